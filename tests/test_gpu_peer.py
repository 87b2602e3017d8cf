"""GPU parity: peer-cache fill (the cache spans GPUs).

Two caches on one device stand in for two GPUs (same protocol, the copy goes
HBM->HBM instead of over NVLink): cache B attaches cache A as a peer and must
return exactly the bytes pread returns (oracle), taking pages from A only when
A holds the same host file at the same close-to-open version, clean and
host-verified. A separate process maps A through CUDA IPC.
"""
import json
import os
import subprocess
import sys
import textwrap

import numpy as np
import pytest

import gen
import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(600)]
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def g():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    g.build.build()
    return g


def whole_pages(P, size):
    offs = np.arange(0, size, P, dtype=np.uint64)
    return offs, np.full(len(offs), P, dtype=np.uint64)


def check_calls(path, size, offs, lens, ret, dst, dstoff):
    for i, (o, l) in enumerate(zip(offs.tolist(), lens.tolist())):
        exp = oracle.pread(path, size, o, l)
        assert ret[i] == len(exp), (i, ret[i], len(exp))
        assert dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes() == exp, i


@pytest.mark.parametrize("P", [65536, 1 << 21])
def test_peer_fill_read_only(g, shmdir, P):
    size = 37 * P + 1111
    path = gen.splitmix_file(os.path.join(shmdir, "ro.bin"), size, seed=11)
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A, \
            g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B:
        B.attach_peer(A.export())
        s, err = A.seqread(path, size - size % 8, P, grid=8)
        assert err == 0 and s == oracle.checksum(path, 0, size - size % 8)
        B.stats(reset=True)
        offs, lens = gen.random_calls(5, 300, size, 3 * P, page_size=P)
        ret, dst, dstoff = B.gread_calls(path, offs, lens, grid=16)
        check_calls(path, size, offs, lens, ret, dst, dstoff)
        st = B.stats()
        npages = (size + P - 1) // P
        assert st["rpc_read"] == 0, st          # every page came from the peer
        assert 0 < st["peer_fill"] <= npages
        assert st["timeout"] == 0 and st["enomem"] == 0


def test_peer_version_mismatch_goes_to_host(g, shmdir):
    """A caches v1 of a file; the file is rewritten through a third cache (version
    bump); B (opened after) must read v2 from the host, never A's stale frames."""
    P = 65536
    path = os.path.join(shmdir, "vm.bin")
    v1 = np.random.default_rng(1).integers(1, 256, size=9 * P + 7, dtype=np.uint8).tobytes()
    v2 = np.random.default_rng(2).integers(1, 256, size=9 * P + 7, dtype=np.uint8).tobytes()
    open(path, "wb").write(v1)
    with g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A, \
            g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B, \
            g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as W:
        B.attach_peer(A.export())
        offs, lens = whole_pages(P, len(v1))
        ret, dst, dstoff = A.gread_calls(path, offs, lens, grid=4)
        assert dst[:len(v1)].tobytes() == v1
        ret = W.gwrite_calls(path, [0], [len(v2)], v2, grid=1)
        assert ret[0] == len(v2) and W.gfsync(path) == 0
        assert open(path, "rb").read() == v2
        B.stats(reset=True)
        ret, dst, dstoff = B.gread_calls(path, offs, lens, grid=4)
        assert dst[:len(v2)].tobytes() == v2
        st = B.stats()
        assert st["peer_fill"] == 0 and st["rpc_read"] > 0, st


def test_peer_fill_from_writer_cache(g, shmdir):
    """A writes a file (O_GWRONCE) and gfsyncs it: pages written from byte 0 without
    holes are host-verified and serve B; the page with a hole goes to the host."""
    P = 65536
    path = os.path.join(shmdir, "w.bin")
    full = np.random.default_rng(3).integers(1, 256, size=6 * P, dtype=np.uint8).tobytes()
    tail = b"\x07" * 100  # page 6: bytes [100, 200) only (hole at [0, 100))
    with g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A, \
            g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B:
        B.attach_peer(A.export())
        fd = A.pin(path, flags=1)  # one incarnation across the write and the sync
        assert fd >= 0
        ret = A.gwrite_calls(path, [0, 6 * P + 100], [6 * P, 100], full + tail, grid=2)
        assert list(ret) == [6 * P, 100]
        assert A.gfsync(path) == 0
        assert A.unpin(fd) == 0
        host = open(path, "rb").read()
        assert host == full + b"\x00" * 100 + tail
        size = len(host)
        B.stats(reset=True)
        offs, lens = whole_pages(P, size)
        ret, dst, dstoff = B.gread_calls(path, offs, lens, grid=4)
        check_calls(path, size, offs, lens, ret, dst, dstoff)
        st = B.stats()
        assert st["peer_fill"] == 6 and st["rpc_read"] == 1, st


def test_peer_fill_under_peer_eviction(g, shmdir):
    """A's cache is smaller than the file (it evicted most pages): B gets the
    pages A still holds from A and the rest from the host, bytes exact."""
    P = 65536
    size = 48 * P + 5
    path = gen.splitmix_file(os.path.join(shmdir, "ev.bin"), size, seed=13)
    with g.GpuFS(cache_bytes=12 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A, \
            g.GpuFS(cache_bytes=16 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B:
        # B: 4 blocks hold up to 3 pages each (2P spans): 16 frames keep the
        # deadlock guard's bound (frames >= blocks x pages held) with slack
        B.attach_peer(A.export())
        s, err = A.seqread(path, size - size % 8, P, grid=4)
        assert err == 0
        B.stats(reset=True)
        offs, lens = gen.random_calls(6, 400, size, 2 * P, page_size=P)
        ret, dst, dstoff = B.gread_calls(path, offs, lens, grid=4)
        check_calls(path, size, offs, lens, ret, dst, dstoff)
        st = B.stats()
        assert st["peer_fill"] > 0 and st["rpc_read"] > 0 and st["evict"] > 0, st


def test_attach_rejects_bad_peers(g):
    P = 65536
    with g.GpuFS(cache_bytes=8 * P, page_size=P, daemon_threads=1) as A, \
            g.GpuFS(cache_bytes=8 * P, page_size=2 * P, daemon_threads=1) as C:
        with pytest.raises(g.GfsError):
            A.attach_peer(A.export())   # itself
        with pytest.raises(g.GfsError):
            A.attach_peer(C.export())   # page size differs
        with pytest.raises(g.GfsError):
            A.attach_peer(b"\x00" * len(C.export()))  # not a descriptor


CHILD = textwrap.dedent("""
    import os, sys, time
    sys.path.insert(0, sys.argv[1])
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    path, size, P, ready, done = sys.argv[2], int(sys.argv[3]), int(sys.argv[4]), sys.argv[5], sys.argv[6]
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A:
        s, err = A.seqread(path, size - size % 8, P, grid=8)
        assert err == 0
        open(ready + ".tmp", "wb").write(A.export())
        os.rename(ready + ".tmp", ready)
        t0 = time.time()
        while not os.path.exists(done) and time.time() - t0 < 300:
            time.sleep(0.05)
""")


def test_peer_fill_across_processes_ipc(g, shmdir):
    """The peer is another process: its cache is mapped through CUDA IPC."""
    P = 65536
    size = 21 * P + 77
    path = gen.splitmix_file(os.path.join(shmdir, "ipc.bin"), size, seed=17)
    ready, done = os.path.join(shmdir, "ready"), os.path.join(shmdir, "done")
    child = subprocess.Popen([sys.executable, "-c", CHILD, ROOT, path, str(size), str(P), ready, done])
    try:
        import time
        t0 = time.time()
        while not os.path.exists(ready):
            assert child.poll() is None, "exporter died"
            assert time.time() - t0 < 300
            time.sleep(0.05)
        with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B:
            B.attach_peer(open(ready, "rb").read())
            offs, lens = whole_pages(P, size)
            ret, dst, dstoff = B.gread_calls(path, offs, lens, grid=8)
            check_calls(path, size, offs, lens, ret, dst, dstoff)
            st = B.stats()
            assert st["peer_fill"] == len(offs) and st["rpc_read"] == 0, st
    finally:
        open(done, "w").close()
        child.wait(timeout=120)
    assert child.returncode == 0


def _c5_rank(rank, ws, port, root, size, iters, outdir):
    """One rank of the C5 pipeline with peer caches (bench.py c5_phase at N = 2):
    write f_r + gfsync, barrier, re-read f_{r+1} (first pass from the writer's
    cache through CUDA IPC), barrier; both ranks share cuda:0 here."""
    import socket  # noqa: F401
    import torch
    import torch.distributed as dist
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=ws)
    P = 1 << 21
    mine, peer = f"{root}/f_{rank}.bin", f"{root}/f_{(rank + 1) % ws}.bin"
    res = {"ok": True, "peer_fill": 0, "rpc_read": 0}
    with g.GpuFS(cache_bytes=64 * P, page_size=P, daemon_threads=2, max_batch=8, timeout_ms=30000) as fs:
        descs = [None] * ws
        dist.all_gather_object(descs, fs.export())
        for r, d in enumerate(descs):
            if r != rank:
                fs.attach_peer(d)
        for it in range(iters):
            data = np.random.default_rng(100 * it + rank).integers(0, 256, size=size, dtype=np.uint8)
            src = torch.from_numpy(data).cuda()
            res["ok"] &= fs.seqwrite(mine, src, chunk=P, grid=8, sync_grid=2) == 0
            dist.barrier()
            want = oracle.checksum(peer, 0, size)
            for _ in range(2):
                s, err = fs.seqread(peer, size, P, grid=8)
                res["ok"] &= err == 0 and s == want
            dist.barrier()
        st = fs.stats()
        res["peer_fill"], res["rpc_read"] = st["peer_fill"], st["rpc_read"]
        dist.barrier()  # no rank unmaps a cache another still reads
    with open(os.path.join(outdir, f"r{rank}.json"), "w") as f:
        json.dump(res, f)
    dist.destroy_process_group()


def test_c5_world2_peer_pipeline(shmdir):
    import socket
    import torch.multiprocessing as mp
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    size, iters = 5 * (1 << 21) + 4096, 3
    mp.spawn(_c5_rank, args=(2, port, shmdir, size, iters, shmdir), nprocs=2, join=True)
    for r in range(2):
        res = json.load(open(os.path.join(shmdir, f"r{r}.json")))
        assert res["ok"], res
        # every first re-read of an iteration comes from the writer's cache
        assert res["peer_fill"] == iters * 6 and res["rpc_read"] == 0, res
