"""Pins for the grep -w oracle.

* hand-derived golden case (tests/golden/grep_hand.json);
* brute-force literal definition on tiny random corpora (orc_grep_brute is a
  second, independent implementation: one word at a time, boundary test per
  occurrence — the paper's own one-word-per-thread formulation);
* GNU grep -owF under LC_ALL=C (secondary: a library routine);
* dictionary format errors (reading R13).
"""
import json
import os
import shutil
import subprocess
from collections import Counter

import numpy as np
import pytest

import gen
import oracle

GOLD = os.path.join(os.path.dirname(__file__), "golden")


def test_hand_golden(shmdir):
    g = json.load(open(os.path.join(GOLD, "grep_hand.json")))
    paths = []
    for i, h in enumerate(g["files_hex"]):
        p = os.path.join(shmdir, f"h{i}.txt")
        open(p, "wb").write(bytes.fromhex(h))
        paths.append(p)
    gen.write_dict(os.path.join(shmdir, "d.bin"), [w.encode() for w in g["words"]])
    gen.write_list(os.path.join(shmdir, "l.txt"), paths)
    for fn in (oracle.grep, oracle.grep_brute):
        r = fn(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"))
        assert r.records.tolist() == g["expected_records"]
        assert r.totals.tolist() == g["expected_totals"]
        assert r.hits.tolist() == g["expected_hits"]


def _same(a, b):
    assert a.records.tolist() == b.records.tolist()
    assert a.totals.tolist() == b.totals.tolist()
    assert a.digest == b.digest
    assert a.hits.tolist() == b.hits.tolist()


@pytest.mark.parametrize("seed", list(range(12)))
def test_tokenising_equals_brute_force(shmdir, seed):
    extra = [b"", b"ab", b"b" * 32 + b" " + b"b" * 33, b"a" * 40]
    c = gen.tiny_corpus(shmdir, seed, nfiles=5, max_bytes=2500, nwords=10, extra_files=extra,
                        extra_words=[b"b" * 32, b"ab", b"ab"])
    _same(oracle.grep(c["dict"], c["list"]), oracle.grep_brute(c["dict"], c["list"]))


def test_threads_do_not_change_result(shmdir):
    c = gen.tiny_corpus(shmdir, 77, nfiles=9, max_bytes=4000, nwords=8)
    _same(oracle.grep(c["dict"], c["list"], nthreads=1), oracle.grep(c["dict"], c["list"], nthreads=4))


@pytest.mark.skipif(shutil.which("grep") is None, reason="no GNU grep")
def test_gnu_grep_secondary_pin(shmdir):
    c = gen.c1_corpus(os.path.join(shmdir, "c1"), seed=5, nfiles=3, file_bytes=40000, nwords=64)
    r = oracle.grep(c["dict"], c["list"], want_hits=False)
    words = [open(c["dict"], "rb").read()[32 * k:32 * k + 32].rstrip(b"\0") for k in range(64)]
    wf = os.path.join(shmdir, "words.txt")
    open(wf, "wb").write(b"\n".join(words) + b"\n")
    env = dict(os.environ, LC_ALL="C")
    for f, p in enumerate(c["paths"]):
        out = subprocess.run(["grep", "-owF", "-f", wf, p], capture_output=True, env=env).stdout
        gnu = Counter(out.split(b"\n")[:-1]) if out else Counter()
        mine = Counter()
        for (ff, k, cnt) in r.records.tolist():
            if ff == f:
                mine[words[k]] = cnt
        assert gnu == mine


def test_c1_shape(shmdir):
    c = gen.c1_corpus(os.path.join(shmdir, "c1"), seed=1, nfiles=2, file_bytes=100000)
    r = oracle.grep(c["dict"], c["list"])
    toks = sum(len(open(p, "rb").read().split()) for p in c["paths"])
    assert r.nfiles == 2 and r.bytes == 200000
    assert 0.002 < int(r.totals.sum()) / toks < 0.2  # dictionary hit density, recipe sanity


@pytest.mark.parametrize("bad", [b"abc", b"\0" * 32, b"ab-c".ljust(32, b"\0"), b"ok".ljust(32, b"\0") + b"x"])
def test_dictionary_format_errors(shmdir, bad):
    d = os.path.join(shmdir, "d.bin")
    open(d, "wb").write(bad)
    gen.write_list(os.path.join(shmdir, "l.txt"), [])
    with pytest.raises(oracle.OracleError):
        oracle.grep(d, os.path.join(shmdir, "l.txt"))


def test_relative_paths_and_blank_lines(shmdir):
    open(os.path.join(shmdir, "a.txt"), "wb").write(b"zz yy zz")
    gen.write_dict(os.path.join(shmdir, "d.bin"), [b"zz"])
    open(os.path.join(shmdir, "l.txt"), "w").write("\n\na.txt\n\n")
    r = oracle.grep(os.path.join(shmdir, "d.bin"), os.path.join(shmdir, "l.txt"))
    assert r.records.tolist() == [[0, 0, 2]]
