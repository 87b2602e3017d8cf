"""GPU parity: gwrite / gfsync / close-to-open, checked with host reads."""
import os

import numpy as np
import pytest

import gen
import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(600)]


@pytest.fixture(scope="module")
def g():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    g.build.build()
    return g


def rnd(n, seed):
    return np.random.default_rng(seed).integers(1, 256, size=n, dtype=np.uint8).tobytes()


def host(p):
    return open(p, "rb").read()


@pytest.mark.parametrize("P", [4096, 65536, 1 << 21])
def test_gwrite_gfsync_visible_on_host(g, shmdir, P):
    path = os.path.join(shmdir, "out.bin")
    size = 5 * P + 333
    data = rnd(size, 1)
    # disjoint writes in random order, several per page, some straddling pages
    rng = np.random.default_rng(2)
    cuts = np.unique(np.concatenate([[0, size], rng.integers(1, size, size=40)]))
    offs, lens = cuts[:-1], np.diff(cuts)
    perm = rng.permutation(len(offs))
    srcoff = offs[perm]
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=4) as fs:
        ret = fs.gwrite_calls(path, offs[perm], lens[perm], data, srcoff=srcoff, grid=8)
        assert (ret == lens[perm]).all()
        assert host(path) == b""                 # not yet synced
        assert fs.gfstat(path, flags=1) == size
        assert fs.gfsync(path) == 0
        assert host(path) == data
        st = fs.stats()
        assert st["writeback"] >= 6 and st["zero_fill"] >= 6


def test_unwritten_bytes_are_zero_and_gread_rejected(g, shmdir):
    path = os.path.join(shmdir, "holes.bin")
    P = 4096
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fs.gwrite_calls(path, [100, 9000], [50, 10], b"\x05" * 50 + b"\x06" * 10)
        assert fs.gfsync(path) == 0
        # gread of a write-once file is -EBADF
        ret, _, _ = fs.gread_calls(path, [0], [10], grid=1)
    h = host(path)
    assert len(h) == 9010
    exp = bytearray(9010)
    exp[100:150] = b"\x05" * 50
    exp[9000:9010] = b"\x06" * 10
    assert h == bytes(exp)


def test_dirty_eviction_then_sync(g, shmdir):
    """Cache of 4 frames, 12 pages written: dirty victims are written back before reuse."""
    path = os.path.join(shmdir, "ev.bin")
    P = 4096
    data = rnd(12 * P, 3)
    with g.GpuFS(cache_bytes=4 * P, page_size=P, max_batch=1, timeout_ms=30000, daemon_threads=2) as fs:
        offs = np.arange(12) * P
        ret = fs.gwrite_calls(path, offs, [P] * 12, data, grid=2)
        assert (ret == P).all()
        assert fs.gfsync(path) == 0
        st = fs.stats()
    assert host(path) == data
    assert st["evict"] >= 8


def test_diff_against_zeros_merge(g, shmdir):
    """A partially written page written back over existing host data keeps the host bytes."""
    path = os.path.join(shmdir, "merge.bin")
    base = rnd(3 * 4096, 4)
    open(path, "wb").write(base)
    with g.GpuFS(cache_bytes=64 * 4096, page_size=4096, timeout_ms=30000, daemon_threads=2) as fs:
        # two disjoint writes per page: the dirty range [lo,hi) has unwritten holes.
        # One block issues all four (with several blocks the file may close and
        # re-open between them, which syncs and starts a new incarnation).
        fs.gwrite_calls(path, [10, 100, 5000, 6000], [20, 20, 30, 5],
                        b"\x01" * 20 + b"\x03" * 20 + b"\x02" * 30 + b"\x04" * 5, grid=1)
        assert fs.gfsync(path) == 0
        hs = fs.host_stats()
    exp = bytearray(base)
    exp[10:30] = b"\x01" * 20
    exp[100:120] = b"\x03" * 20
    exp[5000:5030] = b"\x02" * 30
    exp[6000:6005] = b"\x04" * 5
    assert host(path) == bytes(exp)
    assert hs["merges"] >= 2, hs


def test_close_to_open_between_two_caches(g, shmdir):
    """Workspace model + lazy invalidation on re-open."""
    path = os.path.join(shmdir, "shared.bin")
    old = rnd(50000, 5)
    open(path, "wb").write(old)
    with g.GpuFS(cache_bytes=64 << 20, page_size=4096, timeout_ms=30000, daemon_threads=2) as a, \
            g.GpuFS(cache_bytes=64 << 20, page_size=4096, timeout_ms=30000, daemon_threads=2) as b:
        r, d, _ = a.gread_calls(path, [0], [50000], grid=1)
        assert d[:50000].tobytes() == old
        # reopen without changes keeps the cache
        r, d, _ = a.gread_calls(path, [0], [50000], grid=1)
        sa = a.stats()
        assert sa["reopen_valid"] >= 1 and sa["miss"] == 13
        new = rnd(50000, 6)
        b.gwrite_calls(path, [0], [50000], new)
        assert b.gfsync(path) == 0
        assert host(path) == new
        r, d, _ = a.gread_calls(path, [0], [50000], grid=1)
        assert d[:50000].tobytes() == new
        assert a.stats()["invalidate"] >= 1


def test_gftruncate(g, shmdir):
    path = os.path.join(shmdir, "t.bin")
    open(path, "wb").write(b"x" * 100000)
    with g.GpuFS(cache_bytes=64 << 20, page_size=4096, timeout_ms=30000, daemon_threads=2) as fs:
        assert fs.gftruncate(path, 0) == 0
        assert os.path.getsize(path) == 0
        fs.gwrite_calls(path, [0], [3], b"abc")
        assert fs.gfsync(path) == 0
    assert host(path) == b"abc"


def test_gftruncate_unaligned_clips_the_boundary_page(g, shmdir):
    """Truncate a write-once file held open (its pages dirty in the cache) to a size
    that is not page-aligned: the page the new EOF falls in keeps only its bytes
    below EOF (a later write-back must not grow the file again), the
    pages past it are dropped, and bytes written later past the old EOF leave
    zeros in between."""
    P = 4096
    path = os.path.join(shmdir, "tu.bin")
    data = rnd(3 * P + 100, 7)
    cut = P + 1000
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        fd = fs.pin(path, flags=1)  # held open across the launches: the dirty pages stay this incarnation's
        assert fd >= 0
        assert (fs.gwrite_calls(path, [0], [len(data)], data) == len(data)).all()
        assert fs.gftruncate(path, cut) == 0
        assert os.path.getsize(path) == cut
        assert fs.gfstat(path, flags=1) == cut
        assert fs.gfsync(path) == 0
        assert host(path) == data[:cut]  # the clipped page wrote back [0, cut % P) only
        fs.gwrite_calls(path, [2 * P], [10], b"z" * 10)
        assert fs.gfsync(path) == 0
        assert fs.unpin(fd) == 0
    assert host(path) == data[:cut] + bytes(2 * P - cut) + b"z" * 10


def test_more_files_than_fd_cache(g, shmdir):
    """The daemon's fd cache closes idle host fds and re-opens them by path."""
    paths = []
    for i in range(300):
        p = os.path.join(shmdir, f"f{i}.bin")
        open(p, "wb").write(bytes([i % 251 + 1]) * (100 + i))
        paths.append(p)
    os.environ["GFS_FD_CAP"] = "64"  # read at gfs_init: at most 64 host fds open
    try:
        with g.GpuFS(cache_bytes=64 << 20, page_size=4096, timeout_ms=30000, daemon_threads=2) as fs:
            for rep in range(2):
                for i in (0, 150, 299, 7):
                    pins = [fs.pin(p) for p in paths]  # 300 files open on the GPU at once
                    assert min(pins) >= 0
                    ret, d, _ = fs.gread_calls(paths[i], [0], [1000], grid=1)
                    assert ret[0] == 100 + i and d[:100 + i].tobytes() == bytes([i % 251 + 1]) * (100 + i)
                    for fd in pins:
                        assert fs.unpin(fd) == 0
    finally:
        del os.environ["GFS_FD_CAP"]


@pytest.mark.parametrize("P,sync_grid", [(65536, 1), (65536, 4), (1 << 21, 2)])
def test_c5_write_fsync_reread_iterations(g, shmdir, P, sync_grid):
    """C5 shape on one cache: each iteration gwrites new content from many blocks,
    gfsyncs (from sync_grid blocks), then re-reads the file twice through the same
    cache. The re-open read-only starts a fresh incarnation,
    so every iteration must see its own bytes: host file == source, GPU read-back
    checksum == oracle checksum of the host file."""
    torch = pytest.importorskip("torch")
    path = os.path.join(shmdir, "c5.bin")
    size = 24 * P + 4096  # ragged last page
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=60000, daemon_threads=4,
                 staging_slots=max(64, 32 * sync_grid)) as fs:
        for it in range(3):
            data = np.frombuffer(rnd(size, 100 + it), dtype=np.uint8)
            src = torch.from_numpy(data.copy()).cuda()
            assert fs.seqwrite(path, src, chunk=P // 2 + 16, grid=16, sync_grid=sync_grid) == 0
            assert host(path) == data.tobytes()
            want = oracle.checksum(path, 0, size)
            for _ in range(2):  # cold (fresh incarnation: misses) then warm (hits)
                s, err = fs.seqread(path, size, P, grid=8)
                assert err == 0 and s == want
        st = fs.stats()
    assert st["invalidate"] + st["rpc_open"] >= 3 and st["hit"] > 0
