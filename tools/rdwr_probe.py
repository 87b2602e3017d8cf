"""O_RDWR write-back probe: one cache writes half of every 2 MiB page of a 256 MiB file, then gfsync
from G blocks; prints timings and counters (where the diff write-back spends its time)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_asplos_silbersteinfkw13_b200 as g

P, blk, size = 2 << 20, 64 << 10, 256 << 20
path = "/dev/shm/gfs_rdwr_probe.bin"
orig = np.random.default_rng(1).integers(0, 256, size=size, dtype=np.uint8)
orig.tofile(path)
offs = np.arange(0, size, blk, dtype=np.uint64)[0::2]
data = torch.from_numpy(np.random.default_rng(2).integers(0, 256, size=len(offs) * blk, dtype=np.uint8)).cuda()
for grid in (int(x) for x in os.environ.get("GRIDS", "1 8 64").split()):
    for slots in (int(x) for x in os.environ.get("SLOTS", "0 512").split()):
        orig.tofile(path)
        with g.GpuFS(cache_bytes=2 * size + (256 << 20), page_size=P, daemon_threads=12, max_batch=8,
                     staging_slots=slots) as fs:
            fd = fs.pin(path, flags=g.O_RDWR)
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            fs.gwrite_calls(path, offs, np.full(len(offs), blk, np.uint64), data, grid=296, flags=g.O_RDWR)
            t1 = time.perf_counter()
            fs.stats(reset=True)
            hs0 = fs.host_stats()
            r = fs.gfsync(path, flags=g.O_RDWR, grid=grid)
            t2 = time.perf_counter()
            st = fs.stats()
            hs = fs.host_stats()
            fs.unpin(fd)
        print(f"grid={grid} slots={slots or 'auto'}: gwrite {1e3 * (t1 - t0):.1f} ms, gfsync {1e3 * (t2 - t1):.1f} ms "
              f"(r={r}) writeback={st['writeback']} stage_wait={st['stage_wait']} busy={st['busy']} "
              f"host write busy_ms={(hs['busy_ns'] - hs0['busy_ns']) / 1e6:.1f} merges={hs['merges'] - hs0['merges']}",
              flush=True)
