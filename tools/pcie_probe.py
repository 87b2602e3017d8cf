"""Miss-path kernels for an ncu PCIe-counter pass (pcie__read_bytes: the GPU's
reads of host memory = its pulls of staged / registered pages): a 2 GiB sweep
under a 1 GiB cache through the RPC path, the same with the file registered
(zero-copy), and a 560-row C3 mat-vec. Prints the file bytes each moved."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
GiB = 1 << 30
size, P = 2 * GiB, 2 << 20
path = gen.splitmix_file(f"/dev/shm/gfs_pcie_{size}.bin", size, seed=77)
with g.GpuFS(cache_bytes=GiB, page_size=P, daemon_threads=12, max_batch=1) as fs:
    print("rpc sweep", fs.seqread(path, size, P, grid=296), "file bytes", size, fs.stats()["bytes_h2d"], flush=True)
with g.GpuFS(cache_bytes=GiB, page_size=P, daemon_threads=12, max_batch=1) as fs:
    fs.register_file(path)
    print("zc sweep", fs.seqread(path, size, P, grid=296), "file bytes", size, fs.stats()["bytes_h2d"], flush=True)
m = gen.matrix_files("/dev/shm/gfs_pcie_c3", 560, 131072, seed=3)
with g.GpuFS(cache_bytes=GiB // 8, page_size=P, daemon_threads=12, max_batch=1) as fs:
    y, err = fs.matvec(m["A"], m["x"], "/dev/shm/gfs_pcie_c3/y.f32", 560, 131072)
    print("matvec err", err, "matrix bytes", 560 * 131072 * 4, fs.stats()["bytes_h2d"], flush=True)
