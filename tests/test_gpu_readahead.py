"""GPU parity for NEXT-2 (read-ahead and split-phase reads) and the
fault paths: every byte vs the oracle (pread definition), counters
showing the mechanism ran, and no fill left behind (a full sweep afterwards)."""
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


def _fs(g, **kw):
    kw.setdefault("timeout_ms", 30000)
    kw.setdefault("daemon_threads", 4)
    return g.GpuFS(**kw)


@pytest.mark.parametrize("P,cache_pages,ra,grid,chunk_pages", [
    (65536, 4096, 4, 4, 1),     # cache > file: read-ahead fills, later reads adopt them
    (65536, 48, 8, 8, 1),       # small cache: read-ahead frames compete with the readers' pages
    (4096, 16, 8, 2, 1),        # 16 frames, 2 blocks x (1 + 8): the no-wait allocation gives up
    (1 << 21, 12, 2, 3, 1),     # 2 MiB pages, 24 MiB cache < 40 MiB file
    (65536, 256, 4, 8, 3),      # 3-page calls
])
def test_readahead_sweep_bytes(g, shmdir, P, cache_pages, ra, grid, chunk_pages):
    size = 40 * (1 << 20) + 4321 if P >= (1 << 21) else 300 * P + 999
    path = gen.splitmix_file(os.path.join(shmdir, "ra.bin"), size, seed=31)
    total = size - (size % 8)
    want = oracle.checksum(path, 0, total)
    with _fs(g, cache_bytes=cache_pages * P, page_size=P, readahead=ra, max_batch=4) as fs:
        for rep in range(3):
            s, err = fs.seqread(path, total, chunk_pages * P, grid=grid)
            assert err == 0 and s == want, rep
        st = fs.stats()
        assert st["ra_issued"] > 0
        assert st["ra_adopted"] + st["ra_reaped"] <= st["ra_issued"]
        assert st["timeout"] == 0 and st["enomem"] == 0
        # random calls afterwards (no read-ahead: not sequential) still see exact bytes
        # (grid sized to the deadlock guard: blocks x pages held per call <= frames)
        offs, lens = gen.random_calls(3, 300, size, 2 * P, page_size=P)
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=max(1, min(16, cache_pages // 8)))
        for i, (o, l) in enumerate(zip(offs.tolist(), lens.tolist())):
            exp = oracle.pread(path, size, o, l)
            assert ret[i] == len(exp) and dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes() == exp


def test_readahead_fills_adopted_and_reaped(g, shmdir):
    """One block sweeping a file in page-sized calls: the pages ahead of each call
    are fetched by read-ahead and taken over by the next calls; the ones past the
    last call are completed at gclose (a second sweep then only hits)."""
    P = 65536
    size = 64 * P
    path = gen.splitmix_file(os.path.join(shmdir, "one.bin"), size, seed=32)
    with _fs(g, cache_bytes=256 * P, page_size=P, readahead=4) as fs:
        s, err = fs.seqread(path, size - 8 * P, P, grid=1)
        assert err == 0 and s == oracle.checksum(path, 0, size - 8 * P)
        st = fs.stats(reset=True)
        assert st["ra_adopted"] > 40 and st["ra_reaped"] == 4  # pages 56..59 were fetched ahead, never read
        s, err = fs.seqread(path, size, P, grid=1)
        assert err == 0 and s == oracle.checksum(path, 0, size)
        st = fs.stats()
        assert st["hit"] >= 60  # pages 0..59 cached (the reaped ones published)


def test_split_phase_randread(g, shmdir):
    """K4 with the split-phase lane-parallel gread (gread_lanes_issue / wait, several calls in
    flight per block) == the oracle's sum over the same calls; its raw baseline too."""
    import torch
    P, chunk = 1 << 19, 16384
    size = 64 << 20
    path = gen.splitmix_file(os.path.join(shmdir, "k4.bin"), size, seed=33)
    grid, calls = 64, 48
    offs = (np.random.default_rng(1).integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
    want = oracle.checksum_calls(path, offs, chunk)
    with _fs(g, cache_bytes=size + (16 << 20), page_size=P) as fs:
        assert fs.seqread(path, size, P, grid=32)[1] == 0
        raw = torch.from_file(path, shared=False, size=size, dtype=torch.uint8).cuda()
        for depth in (1, 2, 4):
            for block in (64, 128):
                s, err = fs.randread(path, chunk, offs, grid, block=block, depth=depth)
                assert err == 0 and s == want, (depth, block)
                s, err = fs.randread(None, chunk, offs, grid, block=block, depth=depth, raw=raw)
                assert s == want
        # a cold cache: the split-phase calls' misses are served by the full gread
    with _fs(g, cache_bytes=8 * P, page_size=P) as fs:
        s, err = fs.randread(path, chunk, offs[:16 * 8], 16, block=64, depth=2)
        assert err == 0 and s == oracle.checksum_calls(path, offs[:16 * 8], chunk)


def test_fault_eio_is_reported_and_recovers(g, shmdir):
    """Every 5th READ past page 0 fails on the host: the calls touching those pages
    get -EIO (nothing else changes), no call hangs, and once the fault is gone the
    same calls return the exact bytes (the failed frames are stale, not stuck)."""
    P = 65536
    size = 80 * P + 17
    path = gen.splitmix_file(os.path.join(shmdir, "eio.bin"), size, seed=34)
    offs = (np.arange(80, dtype=np.uint64) * P)
    lens = np.full(80, P, np.uint64)
    with _fs(g, cache_bytes=16 * P, page_size=P, fault=(g.FAULT_EIO << 24) | 5, max_batch=1) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=4)
        st = fs.stats()
        neg = [int(r) for r in ret if r < 0]
        assert neg and all(r == -5 for r in neg), ret  # -EIO
        ok = [i for i, r in enumerate(ret) if r >= 0]
        assert len(ok) + len(neg) == 80
        for i in ok:
            exp = oracle.pread(path, size, int(offs[i]), P)
            assert dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes() == exp
        assert st["timeout"] == 0
        # a full sweep still ends (errors, no hang); staging slots were all given back
        fs.seqread(path, size - (size % 8), P, grid=8)
        assert fs.stats()["timeout"] == 0
    with _fs(g, cache_bytes=16 * P, page_size=P) as fs:
        s, err = fs.seqread(path, size - (size % 8), P, grid=8)
        assert err == 0 and s == oracle.checksum(path, 0, size - (size % 8))


def test_fault_short_read_zero_fills(g, shmdir):
    """A host read that comes back short (as if the file ended there) leaves the
    page's tail zero (R4); every other byte is the file's."""
    P = 65536
    size = 20 * P
    path = gen.splitmix_file(os.path.join(shmdir, "short.bin"), size, seed=35)
    offs = (np.arange(20, dtype=np.uint64) * P)
    lens = np.full(20, P, np.uint64)
    with _fs(g, cache_bytes=64 * P, page_size=P, fault=(g.FAULT_SHORT << 24) | 3, max_batch=1) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=1)
    assert (ret == P).all()
    shorts = 0
    for i in range(20):
        exp = oracle.pread(path, size, i * P, P)
        got = dst[i * P:(i + 1) * P].tobytes()
        if got != exp:
            shorts += 1
            assert got[:P // 2] == exp[:P // 2] and got[P // 2:] == bytes(P // 2), i
    assert shorts > 0


def test_frames_fewer_than_held_pages_enomem(g, shmdir):
    """More pages held at once than frames (4 frames, one block asking for 8 pages in one
    call): -ENOMEM from the deadlock guard, not a hang; the cache works afterwards."""
    P = 65536
    size = 32 * P
    path = gen.splitmix_file(os.path.join(shmdir, "nomem.bin"), size, seed=36)
    with _fs(g, cache_bytes=4 * P, page_size=P, max_batch=8, timeout_ms=20000) as fs:
        ret, dst, dstoff = fs.gread_calls(path, np.array([0], np.uint64), np.array([8 * P], np.uint64), grid=1)
        assert int(ret[0]) == -12, ret  # -ENOMEM
        assert fs.stats()["enomem"] > 0
        ret, dst, dstoff = fs.gread_calls(path, np.array([P], np.uint64), np.array([2 * P], np.uint64), grid=1)
        assert int(ret[0]) == 2 * P and dst[:2 * P].tobytes() == oracle.pread(path, size, P, 2 * P)


@pytest.mark.parametrize("P,cache_pages,ra,grid", [(65536, 4096, 4, 4), (65536, 48, 8, 8), (1 << 21, 12, 2, 3)])
def test_readahead_gmmap_sweep_bytes(g, shmdir, P, cache_pages, ra, grid):
    """Read-ahead behind a sequential gmmap mapper (K1 shape, NEXT-2): the same checksum
    as the oracle with the next pages fetched ahead, in a cache larger and smaller than
    the file; read-ahead fills are posted and adopted or reaped, nothing times out."""
    size = 40 * (1 << 20) + 4321 if P >= (1 << 21) else 300 * P + 999
    path = gen.splitmix_file(os.path.join(shmdir, "ram.bin"), size, seed=37)
    total = size - (size % 8)
    want = oracle.checksum(path, 0, total)
    with _fs(g, cache_bytes=cache_pages * P, page_size=P, readahead=ra, max_batch=4) as fs:
        for rep in range(3):
            s, err = fs.seqread(path, total, P, grid=grid, use_mmap=True)
            assert err == 0 and s == want, rep
        st = fs.stats()
        assert st["ra_issued"] > 0
        assert st["ra_adopted"] + st["ra_reaped"] <= st["ra_issued"]
        assert st["timeout"] == 0 and st["enomem"] == 0
