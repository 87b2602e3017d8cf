"""GPU parity: O_RDWR write sharing with diff-and-merge (
P:L296-315 — a working and a pristine copy per cached page, only the bytes that
differ are written back — and Tab.1 gmsync).

Expected files are the plain definition of workspace consistency with
disjoint writers: the original bytes with every writer's written bytes laid
over them (file extended by the writes); checked with host reads.
"""
import os

import numpy as np
import pytest

import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(600)]
RDWR = 2


@pytest.fixture(scope="module")
def g():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    g.build.build()
    return g


def rnd(n, seed):
    return np.random.default_rng(seed).integers(0, 256, size=n, dtype=np.uint8).tobytes()


def apply(base: bytes, writes):
    out = bytearray(base)
    for o, b in writes:
        if o + len(b) > len(out):
            out.extend(b"\x00" * (o + len(b) - len(out)))
        out[o:o + len(b)] = b
    return bytes(out)


def host(p):
    return open(p, "rb").read()


@pytest.mark.parametrize("P,pinned", [(4096, True), (4096, False), (65536, True)])
def test_rdwr_write_read_sync(g, shmdir, P, pinned):
    path = os.path.join(shmdir, "rw.bin")
    orig = rnd(5 * P + 123, 1)
    open(path, "wb").write(orig)
    rng = np.random.default_rng(2)
    # disjoint writes, some straddling pages, the last one past the old EOF
    offs = sorted(rng.choice(np.arange(0, 5 * P, 97), size=12, replace=False).tolist())
    writes = []
    for k, o in enumerate(offs):
        ln = int(rng.integers(1, 300))
        nxt = offs[k + 1] if k + 1 < len(offs) else o + ln
        ln = max(1, min(ln, nxt - o))
        writes.append((o, rnd(ln, 10 + k)))
    writes.append((len(orig) + 50, rnd(700, 99)))
    data = b"".join(b for _, b in writes)
    woffs = [o for o, _ in writes]
    wlens = [len(b) for _, b in writes]
    want = apply(orig, writes)
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=RDWR) if pinned else None
        ret = fs.gwrite_calls(path, woffs, wlens, data, grid=4, flags=RDWR)
        assert list(ret) == wlens
        if pinned:
            assert host(path) == orig                      # nothing written back yet
            assert fs.gfstat(path, flags=RDWR) == len(want)
        # read back through the cache: own writes over the original bytes
        ro, rl = [0, P - 10, 3 * P + 5], [len(want), 2 * P, 100]
        r, dst, dstoff = fs.gread_calls(path, ro, rl, grid=3, open_flags=RDWR)
        for i, (o, l) in enumerate(zip(ro, rl)):
            exp = want[o:o + l]
            assert r[i] == len(exp)
            assert dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes() == exp, i
        assert fs.gfsync(path, flags=RDWR) == 0
        if pinned:
            assert fs.unpin(fd) == 0
        st = fs.stats()
    assert host(path) == want
    assert st["writeback"] > 0


def test_rdwr_two_writers_share_pages(g, shmdir):
    """Two caches (two GPUs) write interleaved disjoint byte ranges of the same
    pages; each writes back only its changed bytes, so both sets survive (the
    false-sharing case the pristine copy exists for)."""
    P = 4096
    path = os.path.join(shmdir, "share.bin")
    orig = rnd(4 * P, 3)
    open(path, "wb").write(orig)
    wa, wb = [], []
    for k, o in enumerate(range(0, 4 * P, 64)):
        (wa if k % 2 == 0 else wb).append((o + 3, rnd(40, 1000 + k)))
    with g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as A, \
            g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as B:
        fa, fb = A.pin(path, flags=RDWR), B.pin(path, flags=RDWR)
        for fs, ws in ((A, wa), (B, wb)):
            ret = fs.gwrite_calls(path, [o for o, _ in ws], [len(b) for _, b in ws], b"".join(b for _, b in ws),
                                  grid=8, flags=RDWR)
            assert (ret == 40).all()
        assert A.gfsync(path, flags=RDWR, grid=8) == 0  # many blocks share the write-back
        assert B.gfsync(path, flags=RDWR) == 0
        A.unpin(fa)
        B.unpin(fb)
    assert host(path) == apply(orig, wa + wb)
    # the oracle's page-cache model (two caches, same writes) leaves the same file
    q = os.path.join(shmdir, "share_oracle.bin")
    open(q, "wb").write(orig)
    oa, ob = oracle.PageCache(P, 32), oracle.PageCache(P, 32)
    qa, qb = oa.open(q, oracle.PageCache.RDWR), ob.open(q, oracle.PageCache.RDWR)
    for o, b in wa:
        oa.write(qa, o, b)
    for o, b in wb:
        ob.write(qb, o, b)
    oa.fsync(qa)
    ob.fsync(qb)
    assert host(path) == host(q)


def test_rdwr_host_change_not_reverted(g, shmdir):
    """A byte the host (another writer) changes after the GPU fetched the page is
    kept at write-back: only the GPU's own changes are merged."""
    P = 4096
    path = os.path.join(shmdir, "merge.bin")
    orig = rnd(2 * P, 4)
    open(path, "wb").write(orig)
    with g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=RDWR)
        ret = fs.gwrite_calls(path, [100], [50], b"\xAA" * 50, grid=1, flags=RDWR)
        assert ret[0] == 50
        with open(path, "r+b") as f:  # a concurrent writer elsewhere in the same page
            f.seek(1000)
            f.write(b"\x55" * 20)
        assert fs.gfsync(path, flags=RDWR) == 0
        fs.unpin(fd)
    want = apply(orig, [(100, b"\xAA" * 50), (1000, b"\x55" * 20)])
    assert host(path) == want


def test_rdwr_dirty_eviction(g, shmdir):
    """8 frames, 24 pages written: dirty O_RDWR victims (and their pristine
    copies) are diffed back to the host before reuse."""
    P = 4096
    path = os.path.join(shmdir, "ev.bin")
    orig = rnd(24 * P, 5)
    open(path, "wb").write(orig)
    writes = [(p * P + 17, rnd(200, 300 + p)) for p in range(24)]
    with g.GpuFS(cache_bytes=8 * P, page_size=P, max_batch=1, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=RDWR)
        ret = fs.gwrite_calls(path, [o for o, _ in writes], [200] * 24, b"".join(b for _, b in writes), grid=2,
                              flags=RDWR)
        assert (ret == 200).all()
        assert fs.gfsync(path, flags=RDWR) == 0
        fs.unpin(fd)
        st = fs.stats()
    assert host(path) == apply(orig, writes)
    assert st["evict"] >= 8


def test_rdwr_mmap_gmsync(g, shmdir):
    """Writes through gmmap(GFS_PROT_WRITE) pointers reach the host at gmsync
    (Tab.1), merged by diff; later unsynced mapped writes reach it at gfsync;
    a host change in between survives."""
    P = 4096
    path = os.path.join(shmdir, "mm.bin")
    orig = rnd(3 * P, 6)
    open(path, "wb").write(orig)
    w1 = [(10, rnd(100, 1)), (P + 500, rnd(300, 2)), (2 * P + 4000, rnd(96, 3))]
    w2 = [(200, rnd(30, 4)), (P + 900, rnd(10, 5))]
    with g.GpuFS(cache_bytes=32 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=RDWR)
        ret = fs.gwrite_calls(path, [o for o, _ in w1], [len(b) for _, b in w1], b"".join(b for _, b in w1),
                              grid=3, mmap=True, msync=True)
        assert list(ret) == [len(b) for _, b in w1]
        assert host(path) == apply(orig, w1)                 # gmsync wrote them back
        with open(path, "r+b") as f:
            f.seek(3000)
            f.write(b"\x11" * 8)
        ret = fs.gwrite_calls(path, [o for o, _ in w2], [len(b) for _, b in w2], b"".join(b for _, b in w2),
                              grid=2, mmap=True, msync=False)
        assert list(ret) == [len(b) for _, b in w2]
        assert fs.gfsync(path, flags=RDWR) == 0
        fs.unpin(fd)
    assert host(path) == apply(orig, w1 + [(3000, b"\x11" * 8)] + w2)
    q = os.path.join(shmdir, "mm_oracle.bin")
    open(q, "wb").write(orig)
    pc = oracle.PageCache(P, 32)
    qf = pc.open(q, oracle.PageCache.RDWR)
    for o, b in w1:
        pc.mmap_write(qf, o, b, msync=True)
    with open(q, "r+b") as f:
        f.seek(3000)
        f.write(b"\x11" * 8)
    for o, b in w2:
        pc.mmap_write(qf, o, b, msync=False)
    pc.fsync(qf)
    assert host(path) == host(q)


def test_rdwr_mode_rules(g, shmdir):
    P = 4096
    path = os.path.join(shmdir, "modes.bin")
    open(path, "wb").write(rnd(P, 7))
    with g.GpuFS(cache_bytes=16 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=RDWR)
        r, _, _ = fs.gread_calls(path, [0], [10], grid=1)   # O_RDONLY while open O_RDWR: one mode at a time
        assert r[0] == -16                                   # -EBUSY
        ret = fs.gwrite_calls(path, [0], [5], b"hello", grid=1, mmap=True, msync=True)
        assert ret[0] == 5
        fs.unpin(fd)
        ro = os.path.join(shmdir, "ro.bin")
        open(ro, "wb").write(rnd(P, 8))
        # a writable mapping of a file the GPU opened read-only is refused
        fd2 = fs.pin(ro, flags=0)
        ret = fs.gwrite_calls(ro, [0], [5], b"hello", grid=1, mmap=True, msync=True)
        assert ret[0] < 0
        fs.unpin(fd2)
