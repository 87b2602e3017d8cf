"""Diagnose the sequential sweep at several scales (short device timeouts)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import gen, oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g

cases = [  # (file_mib, cache_mib, page_kib, grid, workers)
    (64, 8, 2048, 4, 4),
    (256, 64, 2048, 32, 4),
    (1024, 256, 2048, 64, 8),
    (1024, 256, 2048, 296, 8),
    (1024, 256, 2048, 296, 12),
    (2048, 512, 512, 296, 12),
    (512, 128, 64, 296, 12),
]
if len(sys.argv) > 1:
    cases = [tuple(int(x) for x in a.split(",")) for a in sys.argv[1:]]
g.build.build()
for case in cases:
    fm, cm, pk, grid, w = case[:5]
    sweeps = case[5] if len(case) > 5 else 1
    size = fm << 20
    P = pk << 10
    path = gen.splitmix_file(f"/dev/shm/dbg_{fm}.bin", size, seed=77)
    fs = g.GpuFS(cache_bytes=cm << 20, page_size=P, max_batch=1, daemon_threads=w, timeout_ms=15000)
    t0 = time.time()
    for _ in range(sweeps):
        s, err = fs.seqread(path, size, P, grid=grid)
        if err: break
    dt = time.time() - t0
    st = fs.stats(); hs = fs.host_stats(); info = fs.info()
    ok = (err == 0 and s == oracle.checksum(path, 0, size)) if err == 0 else False
    print(f"file={fm}MiB cache={cm}MiB P={pk}K grid={grid} W={w}: err={err} ok={ok} {dt:.2f}s "
          f"{sweeps*size/dt/1e9:.2f} GB/s x{sweeps} | miss={st['miss']} evict={st['evict']} rpc={st['rpc']} timeout={st['timeout']} "
          f"enomem={st['enomem']} ringwait={st['ring_wait']} | host rpc={hs['rpc']} read={hs['read']} err={hs['errors']} "
          f"pread={hs['bytes_h2d']/max(hs['pread_ns'],1):.2f}GB/s/thr | next={info['host_next_ticket']} tail={info['device_ring_tail']} stage={info['staging_slots']} busy={st['busy']}",
          flush=True)
    fs.close()
