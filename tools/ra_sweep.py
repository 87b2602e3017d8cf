"""Read-ahead (NEXT-2) sweep: sequential gread sweep GB/s against grid size with
and without read-ahead, every page a miss (two files alternate under a smaller
cache); checksums against the oracle."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g

GiB = 1 << 30
size = int(os.environ.get("RA_GIB", "2")) * GiB
paths = [gen.splitmix_file(f"/dev/shm/gfs_ra_{size}_{k}.bin", size, seed=4000 + k) for k in range(2)]
want = [oracle.checksum_mt(p, 0, size) for p in paths]
s = torch.cuda.Stream()
for pk in [int(x) for x in os.environ.get("RA_PAGES", "2048,256,64").split(",")]:
    P = pk << 10
    for grid in [int(x) for x in os.environ.get("RA_GRIDS", "8,32,148,296").split(",")]:
        for ra in [int(x) for x in os.environ.get("RA_RA", "0,2,4,8").split(",")]:
            chunk = max(P, 2 << 20)
            with g.GpuFS(cache_bytes=GiB, page_size=P, daemon_threads=12, readahead=ra,
                         max_batch=min(32, max(1, (8 << 20) // P))) as fs:
                scratch = torch.empty(grid * chunk, dtype=torch.uint8, device="cuda")
                out = torch.zeros(2, dtype=torch.int64, device="cuda")
                ts, ok = [], True
                for rep in range(3):
                    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    out.zero_()
                    with torch.cuda.stream(s):
                        e0.record(s)
                        fs.seqread(paths[rep % 2], size, chunk, grid=grid, stream=s, sync=False, scratch=scratch, out=out)
                        e1.record(s)
                    s.synchronize()
                    ok &= (int(out[0].item()) & ((1 << 64) - 1)) == want[rep % 2] and int(out[1].item()) == 0
                    if rep:
                        ts.append(e0.elapsed_time(e1))
                st = fs.stats()
            ms = float(np.mean(ts))
            print(f"P {pk:5d} KiB grid {grid:4d} readahead {ra}: {size / ms / 1e6:7.2f} GB/s  parity {ok}  "
                  f"ra_issued {st['ra_issued']} adopted {st['ra_adopted']} reaped {st['ra_reaped']} "
                  f"miss {st['miss']} evict {st['evict']}", flush=True)
