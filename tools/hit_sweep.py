"""K4 cache-hit shapes: block-collective gread vs warp-collective gread_warp (and raw TMA baselines)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g

size, P, chunk = 4 << 30, 512 << 10, 16384
total_calls = 1184 * 1024
path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}_r0.bin", size, seed=2000)
rng = np.random.default_rng(7)
offs = (rng.integers(0, size // chunk, size=total_calls) * chunk).astype(np.uint64)
d_off = torch.as_tensor(offs.view(np.int64), device="cuda")
s = torch.cuda.Stream()
with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=12) as fs:
    fs.seqread(path, size, P, grid=296)
    raw = torch.empty(size, dtype=torch.uint8, device="cuda")
    raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8))
    out = torch.zeros(2, dtype=torch.int64, device="cuda")

    def t(fn, reps=5):
        ts = []
        for _ in range(reps + 2):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            with torch.cuda.stream(s):
                out.zero_()
                e0.record(s)
                fn()
                e1.record(s)
            s.synchronize()
            ts.append(e0.elapsed_time(e1))
        return float(np.median(ts[2:])), int(out[0].item()) & ((1 << 64) - 1), int(out[1].item())

    configs = [("block", 1184, 128), ("warp", 148 * 3, 128), ("warp", 148 * 6, 64), ("warp", 148 * 12, 32),
               ("warp", 148, 256), ("warp", 148 * 2, 128)]
    for kind, grid, block in configs:
        calls = total_calls // grid
        n = grid * calls * chunk
        w = kind == "warp"
        mg, sg, eg = t(lambda: fs.randread(path, chunk, d_off[:grid * calls], grid, block=block, stream=s,
                                           sync=False, out=out, warp=w))
        mr, sr, er = t(lambda: fs.randread(None, chunk, d_off[:grid * calls], grid, block=block, raw=raw,
                                           stream=s, sync=False, out=out, warp=w))
        print(f"{kind:5s} grid={grid:5d} block={block:3d} calls={calls:5d}: gpufs {n / mg / 1e6:8.1f} GB/s "
              f"raw {n / mr / 1e6:8.1f} GB/s  ratio {mr / mg:.3f} match={sg == sr} err={eg},{er}", flush=True)
