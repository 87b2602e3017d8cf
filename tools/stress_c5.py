"""Stress the C5 write/sync/re-read loop (test_c5_write_fsync_reread_iterations shape); report diffs."""
import os, sys, tempfile, shutil
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_asplos_silbersteinfkw13_b200 as g

P = int(os.environ.get("P", "65536"))
reps = int(os.environ.get("REPS", "30"))
sync_grid = int(os.environ.get("SYNC_GRID", "1"))
size = 24 * P + 4096
bad = 0
for rep in range(reps):
    d = tempfile.mkdtemp(dir="/dev/shm")
    path = os.path.join(d, "c5.bin")
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=60000, daemon_threads=4,
                 staging_slots=max(64, 32 * sync_grid)) as fs:
        for it in range(3):
            data = np.random.default_rng(100 * rep + it).integers(0, 256, size=size, dtype=np.uint8)
            src = torch.from_numpy(data.copy()).cuda()
            fs.stats(reset=True)
            hs0 = fs.host_stats()
            e = fs.seqwrite(path, src, chunk=P // 2 + 16, grid=16, sync_grid=sync_grid)
            h = np.fromfile(path, dtype=np.uint8)
            if e != 0 or h.size != size or not np.array_equal(h, data):
                bad += 1
                diff = np.nonzero(h[:size] != data[:h.size])[0] if h.size else np.array([])
                runs = []
                if diff.size:
                    start = prev = int(diff[0])
                    for x in diff[1:].tolist() + [None]:
                        if x is None or x != prev + 1:
                            runs.append((start, prev + 1, bool((h[start:prev + 1] == 0).all())))
                            if x is not None:
                                start = x
                        if x is not None:
                            prev = x
                st = fs.stats()
                hs = fs.host_stats()
                print(f"rep {rep} it {it}: err={e} size={h.size} diff runs (start,end,allzero)={runs[:8]} "
                      f"stats={ {k: st[k] for k in ('miss','hit','zero_fill','evict','writeback','busy','retry','locked')} } "
                      f"merges={hs['merges'] - hs0['merges']} mapped={hs['mapped_reads']}", flush=True)
            fs.seqread(path, size, P, grid=8)
    shutil.rmtree(d, ignore_errors=True)
print(f"bad {bad} of {reps * 3}")
