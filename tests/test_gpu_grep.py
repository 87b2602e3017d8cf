"""GPU parity for the grep -w consumer (C1, C4 shapes) vs the oracle: bit-exact
records, totals, hit digest and (C1 / small cases) the full hit list."""
import json
import os

import numpy as np
import pytest

import gen
import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(900)]
GOLD = os.path.join(os.path.dirname(__file__), "golden")


@pytest.fixture(scope="module")
def g():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    g.build.build()
    return g


def compare(got, ref, hits=True):
    assert got["summary"]["err"] == 0, got["summary"]
    assert got["summary"]["nfiles"] == ref.nfiles
    assert got["summary"]["bytes"] == ref.bytes
    assert got["records"].tolist() == ref.records.tolist()
    assert got["totals"].tolist() == ref.totals.tolist()
    assert got["digest"] == ref.digest
    if hits:
        assert got["hits"].tolist() == ref.hits.tolist()


@pytest.mark.parametrize("chunk,P", [(16, 4096), (48, 4096), (4096, 4096), (32768, 65536)])
def test_hand_golden(g, shmdir, chunk, P):
    d = json.load(open(os.path.join(GOLD, "grep_hand.json")))
    paths = []
    for i, hx in enumerate(d["files_hex"]):
        p = os.path.join(shmdir, f"h{i}.txt")
        open(p, "wb").write(bytes.fromhex(hx))
        paths.append(p)
    gen.write_dict(os.path.join(shmdir, "d.bin"), [w.encode() for w in d["words"]])
    gen.write_list(os.path.join(shmdir, "l.txt"), paths)
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        out = fs.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), hits=True, chunk=chunk, grid=8)
    assert out["summary"]["err"] == 0
    assert out["records"].tolist() == d["expected_records"]
    assert out["totals"].tolist() == d["expected_totals"]
    assert out["hits"].tolist() == d["expected_hits"]


@pytest.mark.parametrize("seed", range(6))
def test_tiny_random_vs_oracle(g, shmdir, seed):
    extra = [b"", b"ab", b"b" * 32 + b" " + b"b" * 33, b"a" * 40, b"ab " * 2000]
    c = gen.tiny_corpus(shmdir, seed, nfiles=6, max_bytes=5000, nwords=10, extra_files=extra,
                        extra_words=[b"b" * 32, b"ab", b"ab"])
    ref = oracle.grep_brute(c["dict"], c["list"])
    chunk = [16, 32, 64, 128, 1024, 4096][seed]
    with g.GpuFS(cache_bytes=32 * 4096, page_size=4096, timeout_ms=30000, daemon_threads=2, max_batch=2) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, chunk=chunk, grid=16)
    compare(out, ref)


def test_c1_vs_oracle(g, shmdir):
    c = gen.c1_corpus(os.path.join(shmdir, "c1"), seed=1)
    ref = oracle.grep(c["dict"], c["list"], nthreads=4)
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, timeout_ms=30000, daemon_threads=4) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True)
        out2 = fs.grep(c["dict"], c["list"], hits=True)  # warm: cache reused across launches
        st = fs.stats()
    compare(out, ref)
    compare(out2, ref)
    assert st["reopen_valid"] > 0


def test_c4_shape_small_vs_oracle(g, shmdir):
    c = gen.c4_corpus(os.path.join(shmdir, "c4"), seed=4, nfiles=1500, total_bytes=24 << 20, nwords=58000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=False, nthreads=8)
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, timeout_ms=60000, daemon_threads=8,
                 max_files=4096) as fs:
        out = fs.grep(c["dict"], c["list"], hits=False)
    compare(out, ref, hits=False)
    assert out["summary"]["nhits"] == ref.digest[2]


def test_cache_smaller_than_corpus(g, shmdir):
    """Eviction during grep: a 2 MiB cache under an 8 MiB corpus."""
    c = gen.c1_corpus(os.path.join(shmdir, "c1s"), seed=3, nfiles=8, file_bytes=1 << 20)
    ref = oracle.grep(c["dict"], c["list"], nthreads=4)
    with g.GpuFS(cache_bytes=2 << 20, page_size=64 << 10, timeout_ms=60000, daemon_threads=4, max_batch=1) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, grid=8)
        st = fs.stats()
    compare(out, ref)
    assert st["evict"] > 0


def test_global_file_ids_two_shards(g, shmdir):
    """A shard grepped with file_ids = its global indices reports global files: the
    union of two shards' records, their summed totals and their combined digests
    equal the oracle's over the whole list (hit positions included)."""
    c = gen.c4_corpus(os.path.join(shmdir, "c4s"), seed=14, nfiles=400, total_bytes=4 << 20, nwords=3000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=True)
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    sizes = [os.path.getsize(p) for p in c["paths"]]
    shards = gdist.lpt_shard(sizes, 2)
    recs, tot, dsum, dxor, nh, hits = [], 0, 0, 0, 0, []
    with g.GpuFS(cache_bytes=256 << 20, page_size=65536, timeout_ms=30000, daemon_threads=4, max_files=1024) as fs:
        for r, sh in enumerate(shards):
            lst = gdist.write_shard_list(c["paths"], sh, os.path.join(shmdir, f"shard{r}.txt"))
            out = fs.grep(c["dict"], lst, hits=True, grid=64, file_ids=np.asarray(sh, np.uint32))
            assert out["summary"]["err"] == 0
            recs.append(out["records"])
            tot = tot + out["totals"].astype(object)
            dsum, dxor, nh = (dsum + out["digest"][0]) % (1 << 64), dxor ^ out["digest"][1], nh + out["digest"][2]
            hits.append(out["hits"])
    allr = np.concatenate(recs)
    allr = allr[np.lexsort((allr[:, 1], allr[:, 0]))]
    assert allr.tolist() == ref.records.tolist()
    assert [int(x) for x in tot] == ref.totals.tolist()
    assert (dsum, dxor, nh) == tuple(ref.digest)
    allh = np.concatenate(hits)
    allh = allh[np.lexsort((allh[:, 2], allh[:, 1], allh[:, 0]))]
    assert allh.tolist() == ref.hits.tolist()


def test_warm_reruns_and_keep_open(g, shmdir):
    """Back-to-back runs on one work area (the (file, word) table is left empty by
    each run; keep_open holds files, dictionary and list) stay bit-exact."""
    c = gen.c4_corpus(os.path.join(shmdir, "c4k"), seed=15, nfiles=300, total_bytes=6 << 20, nwords=2000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=False)
    with g.GpuFS(cache_bytes=256 << 20, page_size=65536, timeout_ms=30000, daemon_threads=4, max_files=1024) as fs:
        st = fs.grep_state(c["dict"], c["list"], keep_open=True, chunk=4096)
        for it in range(4):
            out = fs.grep(c["dict"], c["list"], keep_open=True, chunk=4096, state=st)
            compare(out, ref, hits=False)
        s0 = fs.stats()
        out = fs.grep(c["dict"], c["list"], keep_open=True, chunk=4096, state=st)
        compare(out, ref, hits=False)
        assert fs.stats()["rpc_open"] == s0["rpc_open"]  # warm: no open goes to the host


def test_max_chunk_and_rejected_chunk(g, shmdir):
    """The largest item (65472 B: item + halos < 64 KiB, 16-bit token offsets) is
    bit-exact; 65536 is rejected (it overflowed token offsets: wrong counts), and so are
    chunks that are not multiples of 16."""
    c = gen.c4_corpus(os.path.join(shmdir, "c4m"), seed=13, nfiles=120, total_bytes=4 << 20, nwords=2000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=True)
    with g.GpuFS(cache_bytes=256 << 20, page_size=65536, timeout_ms=30000, daemon_threads=4,
                 max_files=1024) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, chunk=65472, grid=64)
        compare(out, ref)
        for bad in (65536, 40):
            with pytest.raises(g.GfsError):
                fs.grep(c["dict"], c["list"], hits=False, chunk=bad, grid=64)


@pytest.mark.parametrize("whole_max", [1, 0, 2 * 4096, 31 * 4096])
def test_whole_file_items_vs_oracle(g, shmdir, whole_max):
    """Multi-chunk files of at most whole_max bytes are one work item (one block
    scans them chunk after chunk, counting in shared memory; most chunks first);
    larger ones are split into chunk items merged through the (file, word) table.
    Every split (1: none whole; 0: 256 KiB; 2 and 31 chunks) is bit-exact, hits included."""
    c = gen.c4_corpus(os.path.join(shmdir, "c4w"), seed=21, nfiles=400, total_bytes=12 << 20, nwords=3000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=True)
    with g.GpuFS(cache_bytes=256 << 20, page_size=65536, timeout_ms=30000, daemon_threads=4,
                 max_files=1024) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, chunk=4096, whole_max=whole_max)
    compare(out, ref)


def test_whole_file_count_table_spill(g, shmdir):
    """A whole multi-chunk file with more distinct dictionary words than the
    per-block count table (at most 4096 slots) spills to the (file, word) table; its
    records are then all merged there: still bit-exact."""
    lex = gen.lexicon(6000, 7, min_len=3, max_len=12, mean=7)
    rng = np.random.default_rng(7)
    body = b" ".join(lex[i] for i in rng.permutation(len(lex)))
    body = body + b"\n" + b" ".join(lex[i] for i in rng.integers(0, len(lex), 4000))
    p0, p1 = os.path.join(shmdir, "big.txt"), os.path.join(shmdir, "small.txt")
    open(p0, "wb").write(body)
    open(p1, "wb").write(b" ".join(lex[:50]))
    gen.write_dict(os.path.join(shmdir, "d.bin"), lex)
    gen.write_list(os.path.join(shmdir, "l.txt"), [p0, p1])
    ref = oracle.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), want_hits=True)
    assert len(body) <= 31 * 4096 and (ref.records[:, 0] == 0).sum() > 4096
    with g.GpuFS(cache_bytes=64 << 20, page_size=65536, timeout_ms=30000, daemon_threads=2) as fs:
        out = fs.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), hits=True, chunk=4096,
                      whole_max=31 * 4096, grid=4)
    compare(out, ref)


def test_grep_cuda_graph_replays(g, shmdir):
    """The grep run captured as a CUDA graph (gfs_grep_graph_create) and replayed:
    every replay equals the oracle (records, totals, digest, the full hit list on C1;
    a C4-shape corpus with files kept open across replays), like direct calls."""
    c = gen.c1_corpus(os.path.join(shmdir, "c1g"), seed=5)
    ref = oracle.grep(c["dict"], c["list"], nthreads=4)
    c4 = gen.c4_corpus(os.path.join(shmdir, "c4g"), seed=16, nfiles=300, total_bytes=6 << 20, nwords=2000)
    ref4 = oracle.grep(c4["dict"], c4["list"], want_hits=False)
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, timeout_ms=30000, daemon_threads=4, max_files=1024) as fs:
        st = fs.grep_state(c["dict"], c["list"], hits=True)
        fs.grep_graph(st, c["dict"], c["list"])
        for _ in range(3):
            compare(fs.grep(c["dict"], c["list"], hits=True, state=st), ref)
        fs.close_grep_graph(st)
        st4 = fs.grep_state(c4["dict"], c4["list"], keep_open=True, chunk=4096)
        compare(fs.grep(c4["dict"], c4["list"], keep_open=True, chunk=4096, state=st4), ref4, hits=False)
        fs.grep_graph(st4, c4["dict"], c4["list"])
        for _ in range(3):
            compare(fs.grep(c4["dict"], c4["list"], keep_open=True, chunk=4096, state=st4), ref4, hits=False)
        fs.close_grep_graph(st4)
