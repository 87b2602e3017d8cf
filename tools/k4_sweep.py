"""K4 (cache-hit 16 KiB greads into shared memory, random offsets of a warm
file): the block-collective kernel against the split-phase lane-parallel one
(depth calls in flight per block) and their raw-TMA baselines; checksums
against the oracle. Prints one line per configuration."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g

size = int(os.environ.get("K4_GIB", "4")) << 30
P = 512 << 10
chunk = 16384
path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}.bin", size, seed=2000)
dev = "cuda:0"
s = torch.cuda.Stream()


def timed(fn, reps=5):
    ts = []
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        with torch.cuda.stream(s):
            e0.record(s)
            fn()
            e1.record(s)
        s.synchronize()
        ts.append(e0.elapsed_time(e1))
    return float(np.mean(ts))


with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=12) as fs:
    assert fs.seqread(path, size, P, grid=296)[1] == 0
    raw = torch.empty(size, dtype=torch.uint8, device=dev)
    raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8))
    out = torch.zeros(2, dtype=torch.int64, device=dev)
    configs = [("block", 1184, 128, 0), ("block", 1184, 256, 0)]
    for depth in (1, 2, 4):
        for block in (128, 256):
            for per_sm in (2, 3, 4, 6):
                if 2 * depth * chunk * per_sm <= 220 * 1024:
                    configs.append(("async", 148 * per_sm, block, depth))
    for kind, grid, block, depth in configs:
        calls = (1184 * 1024) // grid
        rng = np.random.default_rng(7)
        offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
        d_off = torch.as_tensor(offs.view(np.int64), device=dev)
        want = oracle.checksum_calls(path, offs, chunk)
        nbytes = grid * calls * chunk
        rg = lambda: (out.zero_(), fs.randread(path, chunk, d_off, grid, block=block, stream=s, sync=False, out=out,
                                               depth=depth))
        rr = lambda: (out.zero_(), fs.randread(None, chunk, d_off, grid, block=block, raw=raw, stream=s, sync=False,
                                               out=out, depth=depth))
        timed(rg, 2)
        mg = timed(rg)
        okg = (int(out[0].item()) & ((1 << 64) - 1)) == want and int(out[1].item()) == 0
        timed(rr, 2)
        mr = timed(rr)
        okr = (int(out[0].item()) & ((1 << 64) - 1)) == want
        print(f"{kind:5s} grid {grid:5d} block {block:3d} depth {depth}: gpufs {nbytes / mg / 1e6:8.1f} GB/s "
              f"raw {nbytes / mr / 1e6:8.1f} GB/s  vs_raw {mr / mg:.3f}  parity {okg and okr}", flush=True)
