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
