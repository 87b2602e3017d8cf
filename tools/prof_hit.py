"""Small K4 cache-hit run (also used under ncu): warm a file, pin it open, then gread
16 KiB chunks into shared memory at random offsets, and the raw-memory baseline.
Env: HIT_GIB, HIT_PAGE_KIB, HIT_GRID, HIT_CALLS, HIT_BLOCK."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g

size = int(os.environ.get("HIT_GIB", "1")) << 30
P = int(os.environ.get("HIT_PAGE_KIB", "512")) << 10
grid, calls, chunk = int(os.environ.get("HIT_GRID", "592")), int(os.environ.get("HIT_CALLS", "256")), 16384
block = int(os.environ.get("HIT_BLOCK", "256"))
path = gen.splitmix_file(f"/dev/shm/gfs_prof_hit_{size}.bin", size, seed=5)
total_calls = int(os.environ.get("HIT_TOTAL", str(grid * calls)))
calls = total_calls // grid
offs = (np.random.default_rng(7).integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
with g.GpuFS(cache_bytes=size + (64 << 20), page_size=P, daemon_threads=8) as fs:
    s, e = fs.seqread(path, size, P, grid=296)
    assert e == 0
    pfd = fs.pin(path)  # keep it open: the profiled kernels' gopen needs no RPC (ncu replays kernels)
    assert pfd >= 0
    raw = torch.as_tensor(np.fromfile(path, dtype=np.uint8), device="cuda")
    d_off = torch.as_tensor(offs.view(np.int64), device="cuda")
    for _ in range(2):
        a = fs.randread(path, chunk, d_off, grid, block=block)
        b = fs.randread(None, chunk, d_off, grid, block=block, raw=raw)
    assert a == b, (a, b)
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(4)]
    ev[0].record(); fs.randread(path, chunk, d_off, grid, block=block); ev[1].record()
    ev[2].record(); fs.randread(None, chunk, d_off, grid, block=block, raw=raw); ev[3].record()
    torch.cuda.synchronize()
    n = grid * calls * chunk
    print(f"grid={grid} block={block} calls={calls} gpufs {n/ev[0].elapsed_time(ev[1])/1e6:.1f} GB/s  "
          f"raw {n/ev[2].elapsed_time(ev[3])/1e6:.1f} GB/s", flush=True)
