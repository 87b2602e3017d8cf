"""Pins for the write-side oracle: gwrite/gfsync/close-to-open.

Expected contents are constructed from the written buffers themselves and
checked with plain host reads (open/read), never with the oracle's own reader.
"""
import os

import numpy as np
import pytest

import oracle


def host_bytes(p):
    with open(p, "rb") as f:
        return f.read()


def rnd(n, seed):
    # strictly nonzero bytes so "diff against zeros" is unambiguous
    return (np.random.default_rng(seed).integers(1, 256, size=n, dtype=np.uint8)).tobytes()


def test_gwronce_write_fsync_visible_on_host(shmdir):
    p = os.path.join(shmdir, "out.bin")
    pc = oracle.PageCache(4096, 16)
    fd = pc.open(p, oracle.PageCache.GWRONCE)
    data = rnd(10000, 1)
    assert pc.write(fd, 0, data) == 10000
    assert host_bytes(p) == b""          # gwrite alone does not reach the host
    pc.close(fd)
    assert host_bytes(p) == b""          # gclose does not write back
    fd = pc.open(p, oracle.PageCache.GWRONCE)  # re-open as GWRONCE: new incarnation, dirty pages synced first
    assert host_bytes(p) == data
    pc.write(fd, 20000, b"\x07" * 10)
    pc.fsync(fd)                         # gfsync
    h = host_bytes(p)
    assert h[:10000] == data and h[10000:20000] == b"\0" * 10000 and h[20000:] == b"\x07" * 10
    assert pc.stats()["writebacks"] >= 3


def test_gread_on_gwronce_is_ebadf(shmdir):
    pc = oracle.PageCache(4096, 4)
    fd = pc.open(os.path.join(shmdir, "o.bin"), oracle.PageCache.GWRONCE)
    with pytest.raises(oracle.OracleError):
        pc.read(fd, 0, 10)


def test_close_to_open_between_two_caches(shmdir):
    """Workspace model: changes are visible to another GPU when it re-opens."""
    p = os.path.join(shmdir, "shared.bin")
    old = rnd(9000, 2)
    open(p, "wb").write(old)
    reader = oracle.PageCache(4096, 16)
    writer = oracle.PageCache(4096, 16)
    rfd = reader.open(p)
    assert reader.read(rfd, 0, 9000) == old
    wfd = writer.open(p, oracle.PageCache.GWRONCE)
    new = rnd(9000, 3)
    writer.write(wfd, 0, new)
    writer.fsync(wfd)
    writer.close(wfd)
    assert host_bytes(p) == new
    assert reader.read(rfd, 0, 9000) == old     # still open: private workspace copy
    reader.close(rfd)
    rfd = reader.open(p)                          # re-open: lazy invalidation
    assert reader.read(rfd, 0, 9000) == new
    # closed and re-opened without an intervening change: cache is reused (no new misses)
    m = reader.stats()["misses"]
    reader.close(rfd)
    rfd = reader.open(p)
    assert reader.read(rfd, 0, 9000) == new and reader.stats()["misses"] == m


def test_diff_against_zeros_merge(shmdir):
    """Partially written dirty page: bytes not written keep the host copy."""
    p = os.path.join(shmdir, "m.bin")
    a = oracle.PageCache(4096, 4)
    b = oracle.PageCache(4096, 4)
    fb = b.open(p, oracle.PageCache.GWRONCE)
    mid = rnd(200, 4)
    b.write(fb, 100, mid)
    b.fsync(fb)
    fa = a.open(p, oracle.PageCache.GWRONCE)
    lo, hi = rnd(100, 5), rnd(100, 6)
    a.write(fa, 0, lo)
    a.write(fa, 300, hi)
    a.fsync(fa)
    assert host_bytes(p) == lo + mid + hi


def test_dirty_eviction_writes_back(shmdir):
    p = os.path.join(shmdir, "e.bin")
    pc = oracle.PageCache(4096, 2)
    fd = pc.open(p, oracle.PageCache.GWRONCE)
    data = rnd(5 * 4096, 7)
    pc.write(fd, 0, data)  # 5 pages through a 2-page cache
    assert pc.stats()["evictions"] == 3
    assert host_bytes(p) == data[:3 * 4096]
    pc.fsync(fd)
    assert host_bytes(p) == data


def test_ftruncate(shmdir):
    p = os.path.join(shmdir, "t.bin")
    open(p, "wb").write(b"x" * 50000)
    pc = oracle.PageCache(4096, 8)
    fd = pc.open(p, oracle.PageCache.GWRONCE)
    pc.ftruncate(fd, 0)
    assert host_bytes(p) == b"" and pc.size(fd) == 0
    pc.write(fd, 0, b"\x01\x02")
    pc.fsync(fd)
    assert host_bytes(p) == b"\x01\x02" and pc.size(fd) == 2


# ---- O_RDWR diff-and-merge (NEXT-4) pinned to the definition of
# workspace consistency with disjoint writers: the original bytes with every
# writer's bytes laid over them (built here from the buffers, read back with
# plain host reads).
def overlay(base: bytes, writes):
    out = bytearray(base)
    for o, b in writes:
        if o + len(b) > len(out):
            out.extend(b"\x00" * (o + len(b) - len(out)))
        out[o:o + len(b)] = b
    return bytes(out)


def test_rdwr_reads_own_writes_and_syncs_only_changes(shmdir):
    p = os.path.join(shmdir, "rw.bin")
    orig = rnd(3 * 4096 + 100, 40)
    open(p, "wb").write(orig)
    pc = oracle.PageCache(4096, 16)
    fd = pc.open(p, oracle.PageCache.RDWR)
    w = [(10, rnd(50, 41)), (4090, rnd(20, 42)), (3 * 4096 + 150, rnd(30, 43))]  # straddle, past EOF
    for o, b in w:
        assert pc.write(fd, o, b) == len(b)
    want = overlay(orig, w)
    assert pc.read(fd, 0, len(want)) == want          # own writes visible before any sync
    assert host_bytes(p) == orig
    with open(p, "r+b") as f:                         # another writer, bytes this cache never wrote
        f.seek(2000)
        f.write(b"\x07" * 9)
    assert pc.fsync(fd) == 0
    assert host_bytes(p) == overlay(want, [(2000, b"\x07" * 9)])


def test_rdwr_two_writers_false_sharing(shmdir):
    p = os.path.join(shmdir, "share.bin")
    orig = rnd(2 * 4096, 44)
    open(p, "wb").write(orig)
    a, b = oracle.PageCache(4096, 8), oracle.PageCache(4096, 8)
    fa, fb = a.open(p, oracle.PageCache.RDWR), b.open(p, oracle.PageCache.RDWR)
    wa = [(o, rnd(16, 100 + o)) for o in range(0, 2 * 4096, 64)]
    wb = [(o + 32, rnd(16, 200 + o)) for o in range(0, 2 * 4096, 64)]
    for o, d in wa:
        a.write(fa, o, d)
    for o, d in wb:
        b.write(fb, o, d)
    assert a.fsync(fa) == 0 and b.fsync(fb) == 0
    assert host_bytes(p) == overlay(orig, wa + wb)


def test_rdwr_eviction_writes_back_diffs(shmdir):
    p = os.path.join(shmdir, "ev.bin")
    orig = rnd(20 * 4096, 45)
    open(p, "wb").write(orig)
    pc = oracle.PageCache(4096, 3)
    fd = pc.open(p, oracle.PageCache.RDWR)
    w = [(k * 4096 + 7, rnd(33, 300 + k)) for k in range(20)]
    for o, d in w:
        pc.write(fd, o, d)
    assert pc.stats()["evictions"] >= 17
    assert pc.fsync(fd) == 0
    assert host_bytes(p) == overlay(orig, w)


def test_rdwr_mmap_write_and_msync(shmdir):
    p = os.path.join(shmdir, "mm.bin")
    orig = rnd(2 * 4096, 46)
    open(p, "wb").write(orig)
    pc = oracle.PageCache(4096, 8)
    fd = pc.open(p, oracle.PageCache.RDWR)
    assert pc.mmap_write(fd, 4000, rnd(200, 47), msync=True) == 96      # prefix of one page
    w1 = [(4000, rnd(200, 47)[:96])]
    assert host_bytes(p) == overlay(orig, w1)                             # gmsync reached the host
    with open(p, "r+b") as f:
        f.seek(3000)
        f.write(b"\x05" * 4)
    assert pc.mmap_write(fd, 3990, b"\x09" * 5, msync=False) == 5
    assert pc.fsync(fd) == 0
    assert host_bytes(p) == overlay(orig, w1 + [(3000, b"\x05" * 4), (3990, b"\x09" * 5)])


def test_rdwr_mode_conflict(shmdir):
    p = os.path.join(shmdir, "m.bin")
    open(p, "wb").write(rnd(100, 48))
    pc = oracle.PageCache(4096, 4)
    pc.open(p, oracle.PageCache.RDWR)
    with pytest.raises(oracle.OracleError):
        pc.open(p, oracle.PageCache.RDONLY)        # one mode at a time while open
    ro = oracle.PageCache(4096, 4)
    fd = ro.open(p, oracle.PageCache.RDONLY)
    with pytest.raises(oracle.OracleError):
        ro.write(fd, 0, b"x")                      # read-only files are never written
    with pytest.raises(oracle.OracleError):
        ro.mmap_write(fd, 0, b"x")                 # nor mapped writable
