"""GPU parity: gread / gmmap through the C ABI vs the oracle (bit-exact).

Inputs: seeded splitmix files and seeded (off, len) call lists from gen/.
Expected values: oracle.pread (the plain pread definition) per call, and
oracle.checksum for sweeps. Runs on a B200 via gpurun.
"""
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


def check_calls(path, size, offs, lens, ret, dst, dstoff):
    for i, (o, l) in enumerate(zip(offs.tolist(), lens.tolist())):
        exp = oracle.pread(path, size, o, l)
        assert ret[i] == len(exp), (i, o, l, ret[i])
        got = dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes()
        assert got == exp, (i, o, l)


@pytest.mark.parametrize("P,cache_pages,batch,grid", [
    (4096, 4096, 32, 64),      # cache larger than file: misses then hits
    (4096, 64, 1, 16),         # tiny cache: heavy miss/evict/refetch churn
    (65536, 32, 2, 8),
    (1 << 21, 8, 1, 4),        # 2 MiB pages, 16 MiB cache < file
])
def test_gread_random_calls(g, shmdir, P, cache_pages, batch, grid):
    size = 3 * (1 << 21) + 12345 if P >= 65536 else 40 * 4096 * 16 + 77
    path = gen.splitmix_file(os.path.join(shmdir, "f.bin"), size, seed=5)
    offs, lens = gen.random_calls(17, 600, size, max(3 * P // 2, 20000), page_size=P)
    with _fs(g, cache_bytes=cache_pages * P, page_size=P, max_batch=batch) as fs:
        for rep in range(2):
            ret, dst, dstoff = fs.gread_calls(path, offs, lens, mode=0, grid=grid)
            check_calls(path, size, offs, lens, ret, dst, dstoff)
        st = fs.stats()
        assert st["timeout"] == 0 and st["enomem"] == 0
        assert st["miss"] > 0
        if cache_pages * P > size:
            assert st["evict"] == 0


def test_gread_hits_after_warm(g, shmdir):
    P = 65536
    size = 200 * P + 5
    path = gen.splitmix_file(os.path.join(shmdir, "w.bin"), size, seed=8)
    with _fs(g, cache_bytes=512 * P, page_size=P) as fs:
        fs.gread_calls(path, [0], [size], grid=1)
        st0 = fs.stats()
        assert st0["miss"] == 201  # one miss per page of the file (O1 invariant)
        offs, lens = gen.random_calls(3, 500, size, 3 * P, page_size=P)
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=64)
        check_calls(path, size, offs, lens, ret, dst, dstoff)
        st1 = fs.stats()
        assert st1["miss"] == st0["miss"] and st1["hit"] > st0["hit"]


def test_gmmap_prefix(g, shmdir):
    P = 16384
    size = 50 * P + 999
    path = gen.splitmix_file(os.path.join(shmdir, "m.bin"), size, seed=9)
    offs, lens = gen.random_calls(4, 400, size, 3 * P, page_size=P)
    with _fs(g, cache_bytes=16 * P, page_size=P, max_batch=1) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, mode=1, grid=8)
    for i, (o, l) in enumerate(zip(offs.tolist(), lens.tolist())):
        m = 0 if (o >= size or l == 0) else min(l, P - o % P, size - o)
        assert ret[i] == m, (o, l, ret[i], m)
        assert dst[int(dstoff[i]):int(dstoff[i]) + m].tobytes() == oracle.pread(path, size, o, m)


def test_gread_into_shared_memory(g, shmdir):
    P = 65536
    size = 64 * P
    path = gen.splitmix_file(os.path.join(shmdir, "s.bin"), size, seed=10)
    offs, lens = gen.random_calls(5, 300, size, 32768, page_size=P)
    lens[0] = 40000  # larger than the shared buffer: rejected, nothing written
    with _fs(g, cache_bytes=128 * P, page_size=P) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, np.minimum(lens, 40000), mode=2, grid=32, smem=32768)
    assert ret[0] == -22
    ok = np.minimum(lens, 40000) <= 32768
    check_calls(path, size, offs[ok], lens[ok], ret[ok], dst, dstoff[ok])


@pytest.mark.parametrize("P", [4096, 65536])
def test_gread_into_shared_memory_coaligned(g, shmdir, P):
    """Destination at off % 16 in shared memory: the TMA path moves the aligned
    middle of every page span, warp 0 the unaligned head and tail bytes."""
    size = 40 * P + 777
    path = gen.splitmix_file(os.path.join(shmdir, "sc.bin"), size, seed=11)
    offs, lens = gen.random_calls(9, 400, size, 3 * P, page_size=P)
    lens = np.minimum(lens, 32768 - 16)
    lens[:8] = [0, 1, 15, 16, 17, 31, 33, 4095]
    offs[:8] = [3, 1, 7, size - 5, P - 3, 2 * P - 16, 13, size - 100]
    offs[8], lens[8] = P - 1, 2  # one byte on each side of a page boundary
    with _fs(g, cache_bytes=24 * P, page_size=P) as fs:  # < file: misses and evictions too
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, mode=3, grid=2, smem=32768)
    check_calls(path, size, offs, lens, ret, dst, dstoff)


@pytest.mark.parametrize("mode,P,cache_pages,grid", [
    # frames >= warps x pages one call holds (the deadlock guard), else < file
    (4, 4096, 4096, 16),    # warp calls, cache larger than the file
    (4, 4096, 40, 1),       # warp calls, cache < file: misses, evictions, refetches
    (4, 65536, 40, 1),
    (5, 4096, 512, 8),      # warp calls into per-warp shared buffers (TMA middle + edges)
    (5, 65536, 40, 2),
])
def test_gread_warp_api(g, shmdir, mode, P, cache_pages, grid):
    """gopen_warp / gread_warp / gclose_warp (the paper's warp-level design
    point): 8 independent warps per block, same bytes as pread."""
    size = 50 * P + 333
    path = gen.splitmix_file(os.path.join(shmdir, "w.bin"), size, seed=13)
    offs, lens = gen.random_calls(17, 500, size, 3 * P, page_size=P)
    if mode == 5:
        lens = np.minimum(lens, 8192 - 16)
    lens[:6] = [0, 1, 15, 17, 4095, 33]
    offs[:6] = [5, size - 1, 3, P - 7, 1, size + 10]
    with _fs(g, cache_bytes=cache_pages * P, page_size=P) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, mode=mode, grid=grid, block=256,
                                          smem=8192 if mode == 5 else 0)
        st = fs.stats()
    check_calls(path, size, offs, lens, ret, dst, dstoff)
    assert st["timeout"] == 0 and st["enomem"] == 0


@pytest.mark.parametrize("locked", [0, 1])
def test_locked_traversal_same_bytes(g, shmdir, locked):
    P = 4096
    size = 300 * P + 1
    path = gen.splitmix_file(os.path.join(shmdir, "l.bin"), size, seed=12)
    offs, lens = gen.random_calls(6, 400, size, 5 * P, page_size=P)
    with _fs(g, cache_bytes=1024 * P, page_size=P, flags=locked) as fs:
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=48)
        st = fs.stats()
        hs = fs.host_stats()
        info = fs.info()
    try:
        check_calls(path, size, offs, lens, ret, dst, dstoff)
    except AssertionError as e:
        raise AssertionError(f"{e} | dev {st} | host {hs} | info {info}")
    if locked:  # every first lookup takes the lock (busy retries may go lock-free)
        assert st["locked"] >= 300
    else:
        assert st["lockfree"] > 0


@pytest.mark.parametrize("P,cache_mb,use_mmap", [(1 << 21, 8, 0), (65536, 4, 0), (1 << 21, 8, 1)])
def test_seqread_sweep_larger_than_cache(g, shmdir, P, cache_mb, use_mmap):
    size = 64 << 20
    path = gen.splitmix_file(os.path.join(shmdir, "seq.bin"), size, seed=21)
    grid = 4 if P == 1 << 21 else 16
    with _fs(g, cache_bytes=cache_mb << 20, page_size=P, max_batch=1) as fs:
        s, err = fs.seqread(path, size, P, use_mmap=bool(use_mmap), grid=grid)
        st = fs.stats()
    assert err == 0
    assert s == oracle.checksum(path, 0, size)
    npages = size // P
    assert st["miss"] == npages and st["evict"] == npages - (cache_mb << 20) // P


def test_randread_smem_checksum(g, shmdir):
    P = 1 << 17
    size = 256 * P
    chunk = 16384
    path = gen.splitmix_file(os.path.join(shmdir, "k4.bin"), size, seed=31)
    grid, calls = 64, 50
    rng = np.random.default_rng(0)
    offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
    expect = sum(oracle.checksum(path, int(o), chunk) for o in offs) % (1 << 64)
    with _fs(g, cache_bytes=512 * P, page_size=P) as fs:
        s, err = fs.randread(path, chunk, offs, grid)
        assert err == 0 and s == expect
        s2, err2 = fs.randread(path, chunk, offs, grid)
        st = fs.stats()
        assert err2 == 0 and s2 == expect
        import torch
        raw = torch.as_tensor(np.fromfile(path, dtype=np.uint8), device="cuda")
        s3, _ = fs.randread(None, chunk, offs, grid, raw=raw)
        assert s3 == expect
        # warp-collective variant (gread_warp per warp, 4 warps per block), and its raw baseline
        s4, err4 = fs.randread(path, chunk, offs, grid, block=128, warp=True)
        assert err4 == 0 and s4 == expect
        s5, _ = fs.randread(None, chunk, offs, grid, block=128, raw=raw, warp=True)
        assert s5 == expect
    assert st["miss"] <= 256


def test_errors(g, shmdir):
    with _fs(g, cache_bytes=64 << 20, page_size=65536) as fs:
        ret, _, _ = fs.gread_calls(os.path.join(shmdir, "missing.bin"), [0], [10], grid=1)
        assert ret[0] == -2  # -ENOENT from the host open
        assert fs.gfstat(os.path.join(shmdir, "missing.bin")) == -2
        p = os.path.join(shmdir, "x.bin")
        gen.splitmix_file(p, 1000, 1)
        assert fs.gfstat(p) == 1000
        ret, _, _ = fs.gread_calls(p, [0, 999, 1000, 5000], [2000, 10, 1, 1], grid=2)
        assert ret.tolist() == [1000, 1, 0, 0]


def test_mapped_reads_and_external_shrink(g, shmdir):
    """Large read-only files are served from a host mapping (same bytes as
    pread); a file shrunk under the mapping while open reads zeros past the
    new end (R4) instead of crashing the daemon (SIGBUS -> pread fallback)."""
    P = 1 << 20
    size = 80 << 20
    path = gen.splitmix_file(os.path.join(shmdir, "big.bin"), size, seed=44)
    offs, lens = gen.random_calls(9, 200, 40 << 20, 3 * P, page_size=P)  # pages >= 40 MiB stay uncached
    with _fs(g, cache_bytes=64 * P, page_size=P) as fs:
        pfd = fs.pin(path)  # stays open: no revalidation on the next gopens
        assert pfd >= 0
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=16)
        check_calls(path, size, offs, lens, ret, dst, dstoff)
        assert fs.host_stats()["mapped_reads"] > 0
        os.truncate(path, 40 << 20)
        ret, dst, dstoff = fs.gread_calls(path, [70 << 20], [2 * P], grid=1)
        assert ret[0] == 2 * P  # the open file's size is the one seen at gopen
        assert not dst[:2 * P].any()
        fs.unpin(pfd)


def test_few_staging_slots_many_missing_pages(g, shmdir):
    """Regression: 64 blocks each missing 16 pages at once with only 32 staging
    slots. A lane must not wait for a slot while its block holds others (that
    hold-and-wait deadlocked until the timeout); it reports the page busy and
    retries after its block has pulled the pages it did get."""
    P = 4096
    size = 64 * 16 * P * 2
    path = gen.splitmix_file(os.path.join(shmdir, "st.bin"), size, seed=21)
    with _fs(g, cache_bytes=4096 * P, page_size=P, staging_slots=32, timeout_ms=10000) as fs:
        for _ in range(2):
            s, err = fs.seqread(path, size, 16 * P, grid=64)
            assert err == 0 and s == oracle.checksum(path, 0, size)
        st = fs.stats()
    assert st["timeout"] == 0 and st["stage_wait"] > 0


@pytest.mark.parametrize("P", [65536, 1 << 21])
def test_zero_copy_registered_file(g, shmdir, P):
    """gfs_register_file: misses of the registered file pull straight from the host
    page cache (no READ RPC); every byte still equals pread (oracle), under
    eviction churn; an unregistered file in the same cache still uses RPCs."""
    size = 40 * P + 777
    path = gen.splitmix_file(os.path.join(shmdir, "zc.bin"), size, seed=41)
    other = gen.splitmix_file(os.path.join(shmdir, "plain.bin"), 5 * P + 3, seed=42)
    os.chmod(path, 0o444)  # a read-only input (read-only registration when the driver allows it)
    with _fs(g, cache_bytes=12 * P, page_size=P) as fs:
        assert fs.register_file(path) in (0, 1)  # 1: registered read-only
        fs.stats(reset=True)
        offs, lens = gen.random_calls(43, 300, size, 3 * P, page_size=P)
        ret, dst, dstoff = fs.gread_calls(path, offs, lens, grid=4)
        for i, (o, l) in enumerate(zip(offs.tolist(), lens.tolist())):
            exp = oracle.pread(path, size, o, l)
            assert ret[i] == len(exp)
            assert dst[int(dstoff[i]):int(dstoff[i]) + len(exp)].tobytes() == exp, i
        s, err = fs.seqread(path, size - size % 8, P, grid=4)
        assert err == 0 and s == oracle.checksum(path, 0, size - size % 8)
        st = fs.stats()
        assert st["zc_fill"] > 0 and st["rpc_read"] == 0 and st["evict"] > 0, st
        ret, dst, dstoff = fs.gread_calls(other, [0], [5 * P + 3], grid=1)
        assert dst[:5 * P + 3].tobytes() == open(other, "rb").read()
        assert fs.stats()["rpc_read"] > 0
    with pytest.raises(g.GfsError):
        with _fs(g, cache_bytes=4 * P, page_size=P) as fs2:
            fs2.register_file(os.path.join(shmdir, "missing.bin"))


def test_randread_hint_checksum_and_no_leaked_references(g, shmdir):
    """gread_hint (each call names the block's next offset; its page is looked up
    and referenced while the current copy flies): same bytes as plain gread, warm
    and in a cache too small to hold the file (hints then miss or get evicted
    before use), and no reference outlives the kernel: a sweep that needs every
    frame of the tiny cache afterwards still completes."""
    P = 1 << 16
    size = 64 * P
    chunk = 16384
    path = gen.splitmix_file(os.path.join(shmdir, "k4h.bin"), size, seed=33)
    other = gen.splitmix_file(os.path.join(shmdir, "k4h2.bin"), size, seed=34)
    grid, calls = 16, 40
    rng = np.random.default_rng(3)
    offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
    offs[5] = offs[4]  # a hint for the page the block already holds
    expect = sum(oracle.checksum(path, int(o), chunk) for o in offs) % (1 << 64)
    with _fs(g, cache_bytes=128 * P, page_size=P) as fs:  # the file fits: warm hits
        assert fs.randread(path, chunk, offs, grid) == (expect, 0)
        assert fs.randread(path, chunk, offs, grid, hint=True) == (expect, 0)
        assert fs.randread(path, chunk, offs, grid, block=128, hint=True) == (expect, 0)
    with _fs(g, cache_bytes=24 * P, page_size=P) as fs:  # 24 frames for 64 pages: churn
        for _ in range(2):
            assert fs.randread(path, chunk, offs, grid, hint=True) == (expect, 0)
        s, err = fs.seqread(other, size, P, grid=24)
        assert err == 0 and s == oracle.checksum(other, 0, size)


def test_speculative_hit_copy_under_churn(g, shmdir):
    """gread's speculative one-page copy (the TMA starts before the reference is
    confirmed, for slots whose fill is known complete): two files alternate
    through a cache of 16 frames for 2 x 48 pages, so slots routinely name
    frames that were evicted and refilled with another file's page (the
    generation check must reject those copies); the checksums over every call
    equal the oracle's, with speculation on and off (GFS_F_NO_SPECULATE), and the
    counters show both accepted speculative hits and misses."""
    P = 1 << 16
    size = 48 * P
    chunk = 16384
    paths = [gen.splitmix_file(os.path.join(shmdir, f"spec{i}.bin"), size, seed=60 + i) for i in range(2)]
    grid, calls = 12, 64
    rng = np.random.default_rng(11)
    offs = [(rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64) for _ in range(2)]
    expect = [sum(oracle.checksum(p, int(o), chunk) for o in of) % (1 << 64) for p, of in zip(paths, offs)]
    for flags in (0, 8):  # 8 = GFS_F_NO_SPECULATE
        with g.GpuFS(cache_bytes=16 * P, page_size=P, timeout_ms=30000, daemon_threads=4, flags=flags) as fs:
            for rep in range(4):
                for i in (0, 1):
                    assert fs.randread(paths[i], chunk, offs[i], grid, block=96) == (expect[i], 0), (flags, rep, i)
            st = fs.stats()
        assert st["miss"] > 0 and st["hit"] > 0 and st["evict"] > 0
