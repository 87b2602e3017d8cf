"""K4 (16 KiB cache-hit greads into shared memory, random offsets of a warm 4 GiB
file, 512 KiB pages) vs its raw-TMA baseline at several block sizes and resident
blocks per SM (same total calls); checksums against the oracle."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g

size = 4 << 30
P = 512 << 10
chunk = 16384
path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}.bin", size, seed=2000)
dev = "cuda:0"
s = torch.cuda.Stream()
total_calls = 1184 * 1024


def timed(fn, reps=5):
    ts = []
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        fn()
        e1.record(s)
        s.synchronize()
        ts.append(e0.elapsed_time(e1))
    return float(np.mean(ts))


flags = int(os.environ.get("K4_FLAGS", "0"))  # 8: GFS_F_NO_SPECULATE (A/B of the speculative hit copy)
with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=12, flags=flags) as fs:
    assert fs.seqread(path, size, P, grid=296)[1] == 0
    raw = torch.empty(size, dtype=torch.uint8, device=dev)
    raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8))
    for block, per_sm in [(128, 8), (96, 10), (64, 12)]:
        grid = 148 * per_sm
        calls = total_calls // grid
        rng = np.random.default_rng(7)
        offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
        want = oracle.checksum_calls(path, offs, chunk)
        d_off = torch.as_tensor(offs.view(np.int64), device=dev)
        res = {}
        for kind in ("gpufs", "raw"):
            out = {}
            def run():
                out["r"] = fs.randread(path if kind == "gpufs" else None, chunk, d_off, grid, block=block,
                                       raw=raw if kind == "raw" else None, stream=s, sync=False)
            run(); s.synchronize()
            ms = timed(run)
            r = fs.randread(path if kind == "gpufs" else None, chunk, d_off, grid, block=block,
                            raw=raw if kind == "raw" else None)
            res[kind] = (grid * calls * chunk / ms / 1e6, r == (want, 0))
        print(f"flags {flags} block {block} x {per_sm}/SM: gpufs {res['gpufs'][0]:.0f} GB/s raw {res['raw'][0]:.0f} GB/s "
              f"ratio {res['gpufs'][0] / res['raw'][0]:.3f} parity {res['gpufs'][1]} {res['raw'][1]}", flush=True)
