"""Cache-hit gread -> global (hit-global phase shape, for ncu): a warm 4 GiB
file, pinned open (the profiled kernel's gopen needs no RPC: ncu replays
kernels, not the host), swept in 2 MiB calls into a 4 GiB destination."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g
size, P = int(os.environ.get("HG_GIB", "4")) << 30, 2 << 20
path = gen.splitmix_file(f"/dev/shm/gfs_prof_hg_{size}.bin", size, seed=6)
with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=8) as fs:
    assert fs.seqread(path, size, P, grid=296)[1] == 0
    assert fs.pin(path) >= 0
    dst = torch.empty(size, dtype=torch.uint8, device="cuda")
    for _ in range(3):
        s, err = fs.seqread(path, size, P, grid=592, scratch=dst, to_global=True)
        assert err == 0
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(2)]
    ev[0].record()
    fs.seqread(path, size, P, grid=592, scratch=dst, to_global=True)
    ev[1].record()
    torch.cuda.synchronize()
    print(f"hit->global {size / ev[0].elapsed_time(ev[1]) / 1e6:.1f} GB/s delivered", flush=True)
