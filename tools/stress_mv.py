"""Stress the mat-vec y write path: many blocks gwrite 4-byte rows into one
page under eviction; report rows missing from the host file.
Env: CACHE_MB, GRID, PAGE_KIB, ROWS, ITERS."""
import os, sys, tempfile
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import gen, oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g
g.build.build()
d = tempfile.mkdtemp(dir="/dev/shm")
rows, cols = int(os.environ.get("ROWS", "40")), 131072
cache = int(os.environ.get("CACHE_MB", "8")) << 20
grid = int(os.environ.get("GRID", "40"))
P = int(os.environ.get("PAGE_KIB", "2048")) << 10
m = gen.matrix_files(d, rows, cols, seed=3, integer=True)
ref = oracle.matvec(m["A"], m["x"], rows, cols, nthreads=4).astype(np.float32)
bad_runs = 0
iters = int(os.environ.get("ITERS", "10"))
for it in range(iters):
    ypath = os.path.join(d, f"y{it}.f32")
    with g.GpuFS(cache_bytes=cache, page_size=P, timeout_ms=60000, daemon_threads=4, max_batch=1) as fs:
        y, err = fs.matvec(m["A"], m["x"], ypath, rows, cols, grid=grid)
        st = fs.stats(); hs = fs.host_stats()
    yd = y.cpu().numpy(); yh = np.fromfile(ypath, dtype="<f4")
    yh = np.concatenate([yh, np.zeros(max(0, rows - len(yh)), np.float32)])
    bad = np.nonzero(yd != yh)[0]
    devbad = np.nonzero(yd != ref)[0]
    if len(bad) or len(devbad):
        bad_runs += 1
        if bad_runs <= 3:
            print(f"  it {it}: err={err} host-bad {bad.tolist()} dev-bad {devbad.tolist()} zero_fill={st['zero_fill']} "
                  f"writeback={st['writeback']} evict={st['evict']} merges={hs['merges']}", flush=True)
print(f"CACHE_MB={cache>>20} GRID={grid} PAGE_KIB={P>>10} ROWS={rows}: bad runs {bad_runs}/{iters}", flush=True)
