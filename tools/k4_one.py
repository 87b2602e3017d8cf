"""One K4 configuration (for ncu): KIND=block|async GRID BLOCK DEPTH."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
size, P, chunk = 4 << 30, 512 << 10, 16384
grid, block, depth = int(os.environ.get("GRID", "296")), int(os.environ.get("BLOCK", "128")), int(os.environ.get("DEPTH", "2"))
path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}.bin", size, seed=2000)
calls = (1184 * 256) // grid
offs = (np.random.default_rng(7).integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=12) as fs:
    assert fs.seqread(path, size, P, grid=296)[1] == 0
    fs.pin(path)  # held open: the profiled kernel's gopen needs no RPC (ncu replays the kernel, not the host)
    d_off = torch.as_tensor(offs.view(np.int64), device="cuda:0")
    for _ in range(3):
        print(fs.randread(path, chunk, d_off, grid, block=block, depth=depth), flush=True)
    print(fs.stats())
