"""GPU parity for the warp-granularity grep scan (gfs_grep_params.scan = 1: one warp
per work item, the text read in place through gmmap_warp) vs the oracle: bit-exact
records, totals, hit digest and the full hit list, across item splits, page sizes
smaller than items, eviction, count-table spills and warm re-runs."""
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


@pytest.mark.parametrize("chunk,P", [(1024, 4096), (8192, 4096), (32768, 65536)])
def test_hand_golden_warp(g, shmdir, chunk, P):
    d = json.load(open(os.path.join(GOLD, "grep_hand.json")))
    paths = []
    for i, hx in enumerate(d["files_hex"]):
        p = os.path.join(shmdir, f"h{i}.txt")
        open(p, "wb").write(bytes.fromhex(hx))
        paths.append(p)
    gen.write_dict(os.path.join(shmdir, "d.bin"), [w.encode() for w in d["words"]])
    gen.write_list(os.path.join(shmdir, "l.txt"), paths)
    with g.GpuFS(cache_bytes=64 * P, page_size=P, timeout_ms=30000, daemon_threads=2) as fs:
        out = fs.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), hits=True, chunk=chunk,
                      grid=8, block=256, scan=1)
    assert out["summary"]["err"] == 0
    assert out["records"].tolist() == d["expected_records"]
    assert out["totals"].tolist() == d["expected_totals"]
    assert out["hits"].tolist() == d["expected_hits"]


@pytest.mark.parametrize("seed", range(6))
def test_tiny_random_vs_brute_warp(g, shmdir, seed):
    """Items of 1-16 KiB over 4 KiB pages (steps, chunks and pages all cross), tokens of
    32 and 33 bytes at every boundary, empty files and duplicate words."""
    extra = [b"", b"ab", b"b" * 32 + b" " + b"b" * 33, b"a" * 40, b"ab " * 2000,
             (b"x" * 1023 + b" ab") * 5, b" " * 1023 + b"b" * 32]
    c = gen.tiny_corpus(shmdir, seed, nfiles=6, max_bytes=20000, nwords=10, extra_files=extra,
                        extra_words=[b"b" * 32, b"ab", b"ab"])
    ref = oracle.grep_brute(c["dict"], c["list"])
    chunk, whole = [(1024, 0), (1024, 1), (2048, 8192), (4096, 0), (8192, 65536), (16384, 1)][seed]
    with g.GpuFS(cache_bytes=32 * 4096, page_size=4096, timeout_ms=30000, daemon_threads=2, max_batch=2) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, chunk=chunk, grid=4, block=256, scan=1, whole_max=whole)
    compare(out, ref)


def test_c1_vs_oracle_warp(g, shmdir):
    c = gen.c1_corpus(os.path.join(shmdir, "c1"), seed=1)
    ref = oracle.grep(c["dict"], c["list"], nthreads=4)
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, timeout_ms=30000, daemon_threads=4) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, chunk=32768, block=256, scan=1)
        out2 = fs.grep(c["dict"], c["list"], hits=True, chunk=32768, block=256, scan=1)  # warm
    compare(out, ref)
    compare(out2, ref)


def test_c4_shape_small_vs_oracle_warp(g, shmdir):
    c = gen.c4_corpus(os.path.join(shmdir, "c4"), seed=4, nfiles=1500, total_bytes=24 << 20, nwords=58000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=False, nthreads=8)
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, timeout_ms=60000, daemon_threads=8,
                 max_files=4096) as fs:
        st = fs.grep_state(c["dict"], c["list"], keep_open=True, chunk=32768, block=256, scan=1)
        for it in range(3):  # cold, then warm re-runs on the same work area
            out = fs.grep(c["dict"], c["list"], keep_open=True, chunk=32768, block=256, scan=1, state=st)
            compare(out, ref, hits=False)
    assert out["summary"]["nhits"] == ref.digest[2]


def test_cache_smaller_than_corpus_warp(g, shmdir):
    """Eviction under the warp scan: a 2 MiB cache under an 8 MiB corpus (each warp holds
    at most two pages)."""
    c = gen.c1_corpus(os.path.join(shmdir, "c1s"), seed=3, nfiles=8, file_bytes=1 << 20)
    ref = oracle.grep(c["dict"], c["list"], nthreads=4)
    with g.GpuFS(cache_bytes=2 << 20, page_size=64 << 10, timeout_ms=60000, daemon_threads=4, max_batch=1) as fs:
        out = fs.grep(c["dict"], c["list"], hits=True, grid=1, block=256, chunk=16384, scan=1)
        st = fs.stats()
    compare(out, ref)
    assert st["evict"] > 0


def test_global_file_ids_two_shards_warp(g, shmdir):
    c = gen.c4_corpus(os.path.join(shmdir, "c4s"), seed=14, nfiles=400, total_bytes=4 << 20, nwords=3000)
    ref = oracle.grep(c["dict"], c["list"], want_hits=True)
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    sizes = [os.path.getsize(p) for p in c["paths"]]
    shards = gdist.lpt_shard(sizes, 2)
    recs, tot, dsum, dxor, nh, hits = [], 0, 0, 0, 0, []
    with g.GpuFS(cache_bytes=256 << 20, page_size=65536, timeout_ms=30000, daemon_threads=4, max_files=1024) as fs:
        for r, sh in enumerate(shards):
            lst = gdist.write_shard_list(c["paths"], sh, os.path.join(shmdir, f"shard{r}.txt"))
            out = fs.grep(c["dict"], lst, hits=True, grid=64, block=256, chunk=16384, scan=1,
                          file_ids=np.asarray(sh, np.uint32))
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


def test_count_table_spill_warp(g, shmdir):
    """A whole-file item (<= 64 KiB) with more distinct dictionary words than a warp's
    count table (2048 slots) spills to the (file, word) table: still bit-exact."""
    lex = gen.lexicon(5000, 7, min_len=3, max_len=9, mean=6)
    rng = np.random.default_rng(7)
    body = b" ".join(lex[i] for i in rng.permutation(len(lex)))[:60000]
    p0, p1 = os.path.join(shmdir, "big.txt"), os.path.join(shmdir, "small.txt")
    open(p0, "wb").write(body)
    open(p1, "wb").write(b" ".join(lex[:50]))
    gen.write_dict(os.path.join(shmdir, "d.bin"), lex)
    gen.write_list(os.path.join(shmdir, "l.txt"), [p0, p1])
    ref = oracle.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), want_hits=True)
    assert (ref.records[:, 0] == 0).sum() > 2048
    with g.GpuFS(cache_bytes=64 << 20, page_size=65536, timeout_ms=30000, daemon_threads=2) as fs:
        out = fs.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"), hits=True, chunk=32768,
                      whole_max=65536, grid=1, block=32, scan=1)
    compare(out, ref)


def test_rejected_params_warp(g, shmdir):
    c = gen.tiny_corpus(shmdir, 3, nfiles=3, max_bytes=3000, nwords=5)
    with g.GpuFS(cache_bytes=64 << 20, page_size=65536, timeout_ms=30000, daemon_threads=2) as fs:
        for kw in (dict(chunk=1536), dict(chunk=2 * 65536), dict(chunk=4096, whole_max=2 * 65536)):
            with pytest.raises(g.GfsError):
                fs.grep(c["dict"], c["list"], hits=False, block=256, scan=1, **kw)
