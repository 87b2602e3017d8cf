"""C4 warm grep: block scan (scan=0) vs warp scan (scan=1), device ms of the whole
pipeline (CUDA events, mean of REPS), each checked against the oracle.
env: C4_FILES, C4_MIB, VARIANTS="scan:chunk:block:whole,..." (whole 0 = default)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g
nf = int(os.environ.get("C4_FILES", "30000")); mib = int(os.environ.get("C4_MIB", "500"))
reps = int(os.environ.get("REPS", "5"))
variants = [tuple(int(x) for x in v.split(":")) for v in
            os.environ.get("VARIANTS", "0:16384:128:0,1:32768:256:0").split(",")]
c = gen.c4_corpus(f"/dev/shm/gfs_bench_c4_{nf}_{mib}", seed=4, nfiles=nf, total_bytes=mib << 20, nwords=58000)
t = time.time()
ref = oracle.grep(c["dict"], c["list"], want_hits=False, nthreads=os.cpu_count())
print(f"oracle {time.time() - t:.1f} s", flush=True)
s = torch.cuda.Stream()
with g.GpuFS(cache_bytes=4 << 30, page_size=64 << 10, daemon_threads=12, max_files=1 << 16) as fs:
    for scan, chunk, block, whole in variants:
        kw = dict(keep_open=True, rec_cap=1 << 24, chunk=chunk, block=block, whole_max=whole, scan=scan)
        st = fs.grep_state(c["dict"], c["list"], **kw)
        out = fs.grep(c["dict"], c["list"], state=st, stream=s, **kw)  # cold for the first variant
        ms = []
        for _ in range(reps):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s)
            fs.grep(c["dict"], c["list"], state=st, stream=s, sync=False, **kw)
            e1.record(s)
            s.synchronize()
            ms.append(e0.elapsed_time(e1))
        out = fs.grep(c["dict"], c["list"], state=st, stream=s, **kw)
        ok = (out["summary"]["err"] == 0 and out["records"].tolist() == ref.records.tolist()
              and out["totals"].tolist() == ref.totals.tolist() and out["digest"] == ref.digest)
        print(f"scan={scan} chunk={chunk} block={block} whole={whole}: warm {np.mean(ms):.3f} +- {np.std(ms):.3f} ms"
              f" parity={ok} err={out['summary']['err']} nitems={out['summary']['nitems']}", flush=True)
        del st
        torch.cuda.empty_cache()
