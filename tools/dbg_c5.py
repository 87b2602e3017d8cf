import os, sys, numpy as np, torch, tempfile
sys.path.insert(0, os.getcwd())
import paper_conf_asplos_silbersteinfkw13_b200 as g, oracle
d = tempfile.mkdtemp(dir="/dev/shm"); path = os.path.join(d, "c5.bin")
P = 65536; size = 24 * P + 4096
with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=20000, daemon_threads=4, staging_slots=64) as fs:
    for it in range(2):
        data = np.random.default_rng(it).integers(1, 256, size=size, dtype=np.uint8)
        fd = fs.pin(path, flags=1)
        print("it", it, "pin", fd, "fstat", fs.gfstat(path, flags=1), flush=True)
        offs = np.arange(0, size, P // 2, dtype=np.uint64); lens = np.minimum(P // 2, size - offs).astype(np.uint64)
        ret = fs.gwrite_calls(path, offs, lens, data.tobytes(), grid=8)
        print("  gwrite rets", sorted(set(ret.tolist()))[:5], flush=True)
        print("  fsync", fs.gfsync(path), flush=True)
        print("  unpin", fs.unpin(fd), flush=True)
        print("  host ok", open(path, "rb").read() == data.tobytes(), flush=True)
        s, err = fs.seqread(path, size, P, grid=8)
        print("  read", err, s == oracle.checksum(path, 0, size), fs.stats()["invalidate"], flush=True)
