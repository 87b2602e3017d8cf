"""C3 mat-vec (11,200 x 131072 fp32 > 2 GiB cache, fresh cache per pass) with gmmap
read-ahead 0 / 1 / 2 pages (NEXT-2); y checked against the float64 oracle."""
import os, sys, statistics
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import gen, oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g
R, C = int(os.environ.get("ROWS", "11200")), 131072
m = gen.matrix_files("/dev/shm/gfs_bench_c3", R, C, seed=3)
ref = oracle.matvec(m["A"], m["x"], R, C, nthreads=os.cpu_count())
s = torch.cuda.Stream()
state = dict(x=torch.empty(C, dtype=torch.float32, device="cuda"), y=torch.empty(R, dtype=torch.float32, device="cuda"),
             err=torch.zeros(2, dtype=torch.int64, device="cuda"))
for ra in (0, 1, 2, 0, 1, 2):
    ts = []
    for rep in range(4):
        with g.GpuFS(cache_bytes=2 << 30, page_size=2 << 20, daemon_threads=12, max_batch=1, readahead=ra) as fs:
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s)
            fs.matvec(m["A"], m["x"], "/dev/shm/gfs_bench_c3/y_ra.f32", R, C, stream=s, sync=False, state=state)
            e1.record(s)
            s.synchronize()
            st = fs.stats()
        if rep:
            ts.append(e0.elapsed_time(e1))
    y = state["y"].cpu().numpy().astype(np.float64)
    rel = float(np.max(np.abs(y - ref) / np.maximum(np.abs(ref), 1e-300)))
    gb = R * C * 4 / (statistics.mean(ts) * 1e6)
    print(f"readahead {ra}: {gb:.2f} GB/s (+- {statistics.pstdev(ts) / statistics.mean(ts) * gb:.2f}) "
          f"miss {st['miss']} ra_issued {st['ra_issued']} adopted {st['ra_adopted']} reaped {st['ra_reaped']} "
          f"err {int(state['err'][0].item())} max_rel {rel:.1e}", flush=True)
