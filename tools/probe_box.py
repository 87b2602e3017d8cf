"""Box fact probe. Prints facts; writes nothing but stdout."""
import ctypes, os, subprocess, time, json
import torch

def sh(c):
    try:
        return subprocess.run(c, shell=True, capture_output=True, text=True, timeout=60).stdout
    except Exception as e:
        return str(e)

print("nproc", os.cpu_count())
print(sh("lscpu | egrep 'Model name|Socket|NUMA node|Thread|Core'"))
print(sh("free -g; df -h /dev/shm /tmp"))
print(sh("nvidia-smi topo -m"))
print(sh("nvidia-smi --query-gpu=name,pci.bus_id,clocks.max.sm,memory.total --format=csv"))
p = torch.cuda.get_device_properties(0)
print("props", p)
cu = ctypes.CDLL("libcuda.so.1")
cu.cuInit(0)
dev = ctypes.c_int(0); cu.cuDeviceGet(ctypes.byref(dev), 0)
def attr(a):
    v = ctypes.c_int(-1); r = cu.cuDeviceGetAttribute(ctypes.byref(v), a, dev); return (r, v.value)
# CU_DEVICE_ATTRIBUTE_CAN_USE_STREAM_MEM_OPS_V1=92, CAN_USE_64_BIT_STREAM_MEM_OPS_V1=93, CAN_USE_STREAM_WAIT_VALUE_NOR=94
# HOST_NATIVE_ATOMIC_SUPPORTED=86 PAGEABLE_MEMORY_ACCESS=88 CAN_FLUSH_REMOTE_WRITES=98 MAX_SHARED_MEMORY_PER_BLOCK_OPTIN=97
for n,a in [("memops",92),("memops64",93),("waitnor",94),("hostNativeAtomic",86),("pageable",88),("flushRemote",98),("smemOptin",97),("l2",38),("sms",16)]:
    print(n, attr(a))
# pinned H2D / D2H
for chunk in [64<<10, 2<<20, 256<<20]:
    n = 256<<20
    h = torch.empty(n, dtype=torch.uint8).pin_memory(); d = torch.empty(n, dtype=torch.uint8, device="cuda")
    s = torch.cuda.Stream()
    best = 1e9; bestd = 1e9
    for it in range(5):
        torch.cuda.synchronize(); t = time.perf_counter()
        with torch.cuda.stream(s):
            for o in range(0, n, chunk):
                d[o:o+chunk].copy_(h[o:o+chunk], non_blocking=True)
        s.synchronize(); best = min(best, time.perf_counter()-t)
        torch.cuda.synchronize(); t = time.perf_counter()
        with torch.cuda.stream(s):
            for o in range(0, n, chunk):
                h[o:o+chunk].copy_(d[o:o+chunk], non_blocking=True)
        s.synchronize(); bestd = min(bestd, time.perf_counter()-t)
    print(f"chunk {chunk>>10}KiB H2D {n/best/1e9:.1f} GB/s D2H {n/bestd/1e9:.1f} GB/s")
# pread from tmpfs
path = "/dev/shm/probe.bin"
sz = 2<<30
with open(path, "wb") as f:
    f.write(os.urandom(64<<20) * (sz // (64<<20)))
fd = os.open(path, os.O_RDONLY)
buf = bytearray(2<<20); mv = memoryview(buf)
t = time.perf_counter(); o = 0
while o < sz:
    o += os.preadv(fd, [mv], o)
dt = time.perf_counter()-t
print(f"pread 1 thread python 2MiB chunks {sz/dt/1e9:.1f} GB/s")
os.close(fd); os.unlink(path)
print(sh("ncu --query-metrics 2>/dev/null | grep -i pcie | head"))
