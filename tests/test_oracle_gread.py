"""Pins for the gread / gmmap / page-cache oracle.

Pinned against things other than the oracle itself:
* the closed-form content of generator files (word j = splitmix64(seed ^ j)),
  computed here from the generator, never from the oracle;
* hand-derived lengths in tests/golden/gread_hand.json;
* counter invariants of a page cache (first pass, second pass, streaming sweep).
"""
import json
import os

import numpy as np
import pytest

import gen
import oracle

GOLD = os.path.join(os.path.dirname(__file__), "golden")


def closed_form_bytes(seed, size, off, n):
    """Bytes [off, off+n) of a splitmix file, from the generator's closed form."""
    if n <= 0:
        return b""
    w0, w1 = off // 8, (off + n + 7) // 8
    words = gen.splitmix_words(seed, w0, w1 - w0).astype("<u8").view(np.uint8)
    s = off - 8 * w0
    return words[s:s + n].tobytes()


@pytest.mark.parametrize("size", [0, 1, 4095, 4096, 65536 + 13, 1 << 20])
def test_pread_matches_closed_form(shmdir, size):
    path = gen.splitmix_file(os.path.join(shmdir, "f.bin"), size, seed=11)
    offs, lens = gen.random_calls(5, 300, size, 70000, page_size=4096)
    for off, ln in zip(offs.tolist(), lens.tolist()):
        got = oracle.pread(path, size, off, ln)
        n = 0 if off >= size else min(ln, size - off)
        assert len(got) == n
        assert got == closed_form_bytes(11, size, off, n)


def test_hand_golden_lengths(shmdir):
    g = json.load(open(os.path.join(GOLD, "gread_hand.json")))
    S, P = g["file_size"], g["page_size"]
    path = gen.splitmix_file(os.path.join(shmdir, "g.bin"), S, seed=3)
    pc = oracle.PageCache(P, 2)
    fd = pc.open(path)
    for c in g["gread"]:
        assert len(oracle.pread(path, S, c["off"], c["len"])) == c["n"]
        got = pc.read(fd, c["off"], c["len"])
        assert len(got) == c["n"]
        assert got == closed_form_bytes(3, S, c["off"], c["n"])
    for c in g["gmmap"]:
        got = pc.mmap_copy(fd, c["off"], c["len"])
        assert len(got) == c["mapped"]
        assert got == closed_form_bytes(3, S, c["off"], c["mapped"])


@pytest.mark.parametrize("P,cap", [(4096, 3), (4096, 64), (65536, 2), (1 << 21, 2)])
def test_page_cache_model_bytes(shmdir, P, cap):
    size = 3 * P + 777 if P >= 65536 else 40 * P + 5
    path = gen.splitmix_file(os.path.join(shmdir, "f.bin"), size, seed=7)
    pc = oracle.PageCache(P, cap)
    fd = pc.open(path)
    assert pc.size(fd) == size
    offs, lens = gen.random_calls(9, 200, size, 3 * P, page_size=P)
    for off, ln in zip(offs.tolist(), lens.tolist()):
        n = 0 if off >= size else min(ln, size - off)
        assert pc.read(fd, off, ln) == closed_form_bytes(7, size, off, n)
    assert pc.stats()["resident"] <= cap


def test_page_cache_counter_invariants(shmdir):
    P, N = 4096, 50
    size = N * P
    path = gen.splitmix_file(os.path.join(shmdir, "f.bin"), size, seed=1)
    # first pass with C >= pages: misses == distinct pages; second pass: no misses
    pc = oracle.PageCache(P, N)
    fd = pc.open(path)
    rng = np.random.default_rng(0)
    touched = set()
    for _ in range(200):
        o = int(rng.integers(0, size)); ln = int(rng.integers(1, 3 * P))
        pc.read(fd, o, ln)
        n = min(ln, size - o)
        touched.update(range(o // P, (o + n - 1) // P + 1))
    assert pc.stats()["misses"] == len(touched)
    pc.read(fd, 0, size)
    m1 = pc.stats()["misses"]
    assert m1 == N
    pc.read(fd, 0, size)
    assert pc.stats()["misses"] == m1 and pc.stats()["evictions"] == 0
    # single-stream sweep with C < N: misses == N, evictions == N - C
    C = 7
    pc2 = oracle.PageCache(P, C)
    fd2 = pc2.open(path)
    for p in range(N):
        pc2.read(fd2, p * P, P)
    st = pc2.stats()
    assert st["misses"] == N and st["evictions"] == N - C and st["resident"] == C


def test_size_snapshot_at_first_open(shmdir):
    """File size reflects the size at the first gopen (Tab.1)."""
    path = os.path.join(shmdir, "grow.bin")
    gen.random_bytes_file(path, 5000, 1)
    pc = oracle.PageCache(4096, 8)
    fd = pc.open(path)
    with open(path, "ab") as f:
        f.write(b"z" * 3000)
    fd2 = pc.open(path)  # already open: shared fd, no re-snapshot
    assert fd2 == fd and pc.size(fd) == 5000
    assert len(pc.read(fd, 4000, 4000)) == 1000


def test_checksum_closed_form(shmdir):
    size = (1 << 20) + 24
    path = gen.splitmix_file(os.path.join(shmdir, "c.bin"), size, seed=99)
    for off, ln in [(0, size), (8, 4096), (4096 * 3, 65536), (size - 16, 16), (0, 0)]:
        w = gen.splitmix_words(99, off // 8, ln // 8).astype(object)
        j = np.arange(off // 8, off // 8 + ln // 8).astype(object)
        expect = int(sum(int(a) * (2 * int(b) + 1) for a, b in zip(w, j)) % (1 << 64)) if ln else 0
        assert oracle.checksum(path, off, ln) == expect


def test_checksum_ragged_bytes(shmdir):
    """Unaligned ranges: bytes outside [off, off+len) count as zero."""
    path = os.path.join(shmdir, "r.bin")
    data = bytes(range(1, 41))
    open(path, "wb").write(data)
    # word 1 = bytes 8..15; take only bytes 10..12 -> value b10<<16 | b11<<24 | b12<<32, weight 3
    expect = (data[10] << 16 | data[11] << 24 | data[12] << 32) * 3
    assert oracle.checksum(path, 10, 3) == expect


def _closed_form_checksum(seed, off, ln):
    """Checksum of bytes [off, off+ln) of a splitmix file from the generator's
    closed form (SURVEY §8(c) O1 pin 3), byte by byte with Python ints."""
    if ln == 0:
        return 0
    w0, w1 = off // 8, (off + ln - 1) // 8
    words = gen.splitmix_words(seed, w0, w1 - w0 + 1)
    s = 0
    for o in range(off, off + ln):
        b = (int(words[o // 8 - w0]) >> (8 * (o % 8))) & 0xFF
        s += (b << (8 * (o % 8))) * (2 * (o // 8) + 1)
    return s % (1 << 64)


def test_checksum_mt_closed_form(shmdir):
    """The threaded split of the checksum equals the closed form for any cut."""
    size = 300_000
    path = gen.splitmix_file(os.path.join(shmdir, "m.bin"), size, seed=5)
    for off, ln in [(0, size), (3, 77_777), (size - 13, 13), (8, 0), (12345, 99_999)]:
        expect = _closed_form_checksum(5, off, ln)
        for t in (1, 2, 3, 7, 16):
            assert oracle.checksum_mt(path, off, ln, nthreads=t) == expect, (off, ln, t)


def test_checksum_calls_closed_form(shmdir):
    """K4 total = sum over calls of the per-call checksum (repeats included)."""
    size = 1 << 18
    path = gen.splitmix_file(os.path.join(shmdir, "k.bin"), size, seed=11)
    rng = np.random.default_rng(3)
    chunk = 4096
    offs = rng.integers(0, size // chunk, size=37) * chunk
    offs[5] = offs[9]  # a repeated call counts twice
    expect = sum(_closed_form_checksum(11, int(o), chunk) for o in offs) % (1 << 64)
    for t in (1, 4):
        assert oracle.checksum_calls(path, offs, chunk, nthreads=t) == expect
    assert oracle.checksum_calls(path, [], chunk) == 0
