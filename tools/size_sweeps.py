"""SURVEY §8(d) size sweeps, one B200, every point checked against the oracle:
  C2: a sequential gread sweep of one splitmix file of S GiB, S in {1,2,4,8,16,32,64}
      (capped by tmpfs), 4 GiB cache, 2 MiB pages, grid 296, a FRESH cache per
      timed sweep (every page a miss), mean +- std of 3; checksum == oracle.checksum_mt.
  C3 (Fig. 8): y = A x for R rows x 131072 fp32, R in {560, 1120, 5600,
      11200, 22400} (280 MiB - 11.2 GiB), 2 GiB cache, 2 MiB pages, fresh cache per
      pass, mean +- std of 3; every row within 1e-5 of the float64 oracle.
Each point is one JSON line; the link peak (copy engine and SM pull) is measured first.
env: C2_SIZES (GiB, comma list), C3_ROWS (comma list), REPS."""
import json, os, shutil, statistics, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g

SHM = "/dev/shm/gfs_sweeps"
os.makedirs(SHM, exist_ok=True)
reps = int(os.environ.get("REPS", "3"))
sizes = [int(x) for x in os.environ.get("C2_SIZES", "1,2,4,8,16,32,64").split(",") if x]
rows_list = [int(x) for x in os.environ.get("C3_ROWS", "560,1120,5600,11200,22400").split(",") if x]
s = torch.cuda.Stream()
nproc = os.cpu_count() or 1


def timed(fn):
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(s)
    fn()
    e1.record(s)
    s.synchronize()
    return e0.elapsed_time(e1)


def mstd(v):
    return statistics.mean(v), (statistics.stdev(v) if len(v) > 1 else 0.0)


ce, sm = g.gfs_probe_h2d(s.cuda_stream)
peak = max(ce or 0, sm or 0) or None
print(json.dumps({"link_peak": {"copy_engine_GBps": ce, "sm_pull_GBps": sm}}), flush=True)

for S in sizes:
    free = shutil.disk_usage("/dev/shm").free
    if (S << 30) + (4 << 30) > free:
        print(json.dumps({"c2_file_gib": S, "skipped": f"tmpfs free {free >> 30} GiB"}), flush=True)
        continue
    path = gen.splitmix_file(f"{SHM}/c2_{S}.bin", S << 30, seed=1000 + S)
    want = oracle.checksum_mt(path, 0, S << 30, nthreads=nproc)
    ts, ok = [], True
    scratch = torch.empty(296 * (2 << 20), dtype=torch.uint8, device="cuda")
    res = torch.zeros(2, dtype=torch.int64, device="cuda")
    for r in range(reps):
        with g.GpuFS(cache_bytes=4 << 30, page_size=2 << 20, daemon_threads=12) as fs:
            t = timed(lambda: (res.zero_(), fs.seqread(path, S << 30, 2 << 20, grid=296, stream=s, sync=False,
                                                       scratch=scratch, out=res)))
            st = fs.stats()
        ok &= (int(res[0].item()) & ((1 << 64) - 1)) == want and int(res[1].item()) == 0
        ts.append(t)
    m, sd = mstd(ts)
    gbps = (S << 30) / (m * 1e6)
    print(json.dumps({"c2_file_gib": S, "GBps": round(gbps, 3), "GBps_std": round(gbps * sd / m, 3),
                      "frac_link_peak": round(gbps / peak, 4) if peak else None, "misses": st["miss"],
                      "parity": bool(ok), "tmpfs_free_gib": free >> 30}), flush=True)
    os.remove(path)
    del scratch

cols = 131072
for R in rows_list:
    root = f"{SHM}/c3_{R}"
    m_ = gen.matrix_files(root, R, cols, seed=3)
    ypath = f"{root}/y.f32"
    state = dict(x=torch.empty(cols, dtype=torch.float32, device="cuda"),
                 y=torch.empty(R, dtype=torch.float32, device="cuda"),
                 err=torch.zeros(2, dtype=torch.int64, device="cuda"))
    ts, miss = [], []
    for r in range(1 + reps):  # pass 0 untimed (process warm-up, not cache)
        with g.GpuFS(cache_bytes=2 << 30, page_size=2 << 20, daemon_threads=12, max_batch=1) as fs:
            t = timed(lambda: fs.matvec(m_["A"], m_["x"], ypath, R, cols, stream=s, sync=False, state=state))
            st = fs.stats()
        if r:
            ts.append(t)
            miss.append(st["miss"])
    ref = oracle.matvec(m_["A"], m_["x"], R, cols, nthreads=nproc)
    y = state["y"].cpu().numpy().astype(np.float64)
    rel = float(np.max(np.abs(y - ref) / np.maximum(np.abs(ref), 1e-300)))
    m, sd = mstd(ts)
    nbytes = R * cols * 4
    gbps = nbytes / (m * 1e6)
    print(json.dumps({"c3_rows": R, "matrix_mib": nbytes >> 20, "GBps": round(gbps, 3),
                      "GBps_std": round(gbps * sd / m, 3), "frac_link_peak": round(gbps / peak, 4) if peak else None,
                      "misses_per_pass": miss, "err": int(state["err"][0].item()),
                      "parity": {"rows_checked": R, "max_rel_err": rel, "ok": rel <= 1e-5}}), flush=True)
    shutil.rmtree(root, ignore_errors=True)
