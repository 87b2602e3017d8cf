"""C4 grep stage timing (GFS_GREP_DEBUG=1 prints per-stage ms)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
g.build.build()
nf = int(os.environ.get("C4_FILES", "30000")); mib = int(os.environ.get("C4_MIB", "500"))
c = gen.c4_corpus(f"/dev/shm/gfs_bench_c4_{nf}_{mib}", seed=4, nfiles=nf, total_bytes=mib << 20, nwords=58000)
with g.GpuFS(cache_bytes=4 << 30, page_size=64 << 10, daemon_threads=12, max_files=1 << 16) as fs:
    for phase in ("cold", "warm"):
        t = time.time()
        out = fs.grep(c["dict"], c["list"], keep_open=True, rec_cap=1 << 24)
        print(phase, f"{(time.time()-t)*1e3:.1f} ms", out["summary"], flush=True)
    print(fs.stats())
    print(fs.host_stats())
