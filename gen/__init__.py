"""Seeded synthetic input generators shared by the oracle tests and the GPU tests.

This module holds NONE of the method's arithmetic (no page lookup, no grep,
no checksum, no mat-vec): it only writes input files to tmpfs. Recipes follow
SURVEY.md §8(d) / DESIGN.md §"Input recipe":

* ``splitmix_file``  — C2 content: the 8-byte little-endian word at byte
  offset o (o % 8 == 0) is ``splitmix64(seed ^ (o // 8))``.
* ``c1_corpus``      — 64-word dictionary drawn uniformly from a 20k-word
  English-like lexicon; 16 files x 512 KiB of Zipf(1.1) text + 10% random
  identifiers (some longer than 32 bytes), spaces / punctuation / newlines.
* ``c4_corpus``      — 58,000-word dictionary ([a-z]{1,28}); ~30,000 C-like
  files, lognormal sizes (mu = ln 7 KiB, sigma = 1.3) clipped to
  [64 B, 4 MiB] and rescaled to the requested total, 3-5 directory levels.
* ``matrix_files``   — C3 row-major fp32 A (R x C) and x (C), U[0,1) or
  small integers.

Everything is deterministic in (recipe, seed, size). Outputs are written to a
temporary name and renamed, with a ``.done`` marker holding the parameters,
so an interrupted generation is never reused.
"""
from __future__ import annotations

import json
import os
import shutil

import numpy as np

SHM = "/dev/shm"
_M64 = np.uint64(0xFFFFFFFFFFFFFFFF)


def splitmix64_np(x: np.ndarray) -> np.ndarray:
    """Vectorised SplitMix64 (Steele et al.) over uint64 — the input generator's PRNG."""
    with np.errstate(over="ignore"):
        z = x.astype(np.uint64) + np.uint64(0x9E3779B97F4A7C15)
        z = (z ^ (z >> np.uint64(30))) * np.uint64(0xBF58476D1CE4E5B9)
        z = (z ^ (z >> np.uint64(27))) * np.uint64(0x94D049BB133111EB)
        return z ^ (z >> np.uint64(31))


def _marker_ok(path: str, params: dict) -> bool:
    m = path + ".done"
    try:
        with open(m) as f:
            return json.load(f) == params
    except Exception:
        return False


def _mark(path: str, params: dict):
    with open(path + ".done", "w") as f:
        json.dump(params, f)


def splitmix_words(seed: int, first_word: int, nwords: int) -> np.ndarray:
    j = np.arange(first_word, first_word + nwords, dtype=np.uint64)
    return splitmix64_np(np.uint64(seed) ^ j)


def splitmix_file(path: str, size: int, seed: int) -> str:
    """C2 file: word j (bytes [8j, 8j+8)) = splitmix64(seed ^ j), truncated to ``size`` bytes."""
    params = {"kind": "splitmix", "size": int(size), "seed": int(seed)}
    if os.path.exists(path) and os.path.getsize(path) == size and _marker_ok(path, params):
        return path
    tmp = path + f".tmp{os.getpid()}"
    chunk_words = 1 << 23  # 64 MiB
    nwords = (size + 7) // 8
    with open(tmp, "wb") as f:
        w = 0
        while w < nwords:
            n = min(chunk_words, nwords - w)
            a = splitmix_words(seed, w, n).astype("<u8").view(np.uint8)
            end = min(size - 8 * w, a.size)
            f.write(a[:end].tobytes())
            w += n
    os.replace(tmp, path)
    _mark(path, params)
    return path


def random_bytes_file(path: str, size: int, seed: int) -> str:
    rng = np.random.default_rng(seed)
    data = rng.integers(0, 256, size=size, dtype=np.uint8)
    with open(path, "wb") as f:
        f.write(data.tobytes())
    return path


# ----------------------------------------------------------------- text corpora
_LETTERS = np.frombuffer(b"abcdefghijklmnopqrstuvwxyz", dtype=np.uint8)
_IDFIRST = np.frombuffer(b"abcdefghijklmnopqrstuvwxyz_", dtype=np.uint8)
_IDREST = np.frombuffer(b"abcdefghijklmnopqrstuvwxyz0123456789_", dtype=np.uint8)


def lexicon(n: int, seed: int, min_len: int = 2, max_len: int = 14, mean: float = 6.5) -> list[bytes]:
    """n distinct lowercase words with an English-like (binomial-ish) length distribution."""
    rng = np.random.default_rng(seed)
    out: list[bytes] = []
    seen: set[bytes] = set()
    span = max_len - min_len
    p = min(max((mean - min_len) / max(span, 1), 0.01), 0.99)
    while len(out) < n:
        m = (n - len(out)) * 2 + 16
        lens = min_len + rng.binomial(span, p, size=m)
        letters = rng.choice(_LETTERS, size=int(lens.sum()))
        pos = 0
        for L in lens:
            w = letters[pos:pos + L].tobytes()
            pos += L
            if w not in seen:
                seen.add(w)
                out.append(w)
                if len(out) == n:
                    break
    return out


def random_identifiers(n: int, rng, max_rest: int = 40) -> list[bytes]:
    """[a-z_][a-z0-9_]{0,max_rest} — some longer than 32 bytes."""
    lens = 1 + rng.integers(0, max_rest + 1, size=n)
    first = rng.choice(_IDFIRST, size=n)
    rest = rng.choice(_IDREST, size=int(lens.sum()))
    out, pos = [], 0
    for i, L in enumerate(lens):
        out.append(bytes([first[i]]) + rest[pos:pos + L - 1].tobytes())
        pos += L - 1
    return out


class _Vocab:
    """Byte strings laid out contiguously, for vectorised gather-assembly of text."""

    def __init__(self, items: list[bytes]):
        self.lens = np.array([len(s) for s in items], dtype=np.int64)
        self.starts = np.concatenate([[0], np.cumsum(self.lens)[:-1]]).astype(np.int64)
        self.buf = np.frombuffer(b"".join(items), dtype=np.uint8)


def _assemble(tok: _Vocab, sep: _Vocab, tok_ids: np.ndarray, sep_ids: np.ndarray) -> np.ndarray:
    """Interleave token[tok_ids[i]] + sep[sep_ids[i]] into one uint8 array."""
    src = np.concatenate([tok.buf, sep.buf])
    off_sep = tok.buf.size
    n = tok_ids.size
    starts = np.empty(2 * n, dtype=np.int64)
    lens = np.empty(2 * n, dtype=np.int64)
    starts[0::2] = tok.starts[tok_ids]
    lens[0::2] = tok.lens[tok_ids]
    starts[1::2] = sep.starts[sep_ids] + off_sep
    lens[1::2] = sep.lens[sep_ids]
    total = int(lens.sum())
    piece_begin = np.concatenate([[0], np.cumsum(lens)[:-1]])
    idx = np.repeat(starts - piece_begin, lens) + np.arange(total, dtype=np.int64)
    return src[idx]


def _zipf_ids(rng, n_vocab: int, size: int, s: float) -> np.ndarray:
    ranks = np.arange(1, n_vocab + 1, dtype=np.float64)
    p = ranks ** (-s)
    cdf = np.cumsum(p)
    cdf /= cdf[-1]
    return np.minimum(np.searchsorted(cdf, rng.random(size)), n_vocab - 1)


def text_stream(nbytes: int, rng, tok: _Vocab, tok_weights_sampler, sep: _Vocab, sep_p: np.ndarray) -> np.ndarray:
    """Generate >= nbytes of text and cut to exactly nbytes."""
    parts, have = [], 0
    avg = float(tok.lens.mean() + (sep.lens * sep_p).sum())
    while have < nbytes:
        n = int((nbytes - have) / avg * 1.05) + 64
        n = min(n, 4_000_000)
        tid = tok_weights_sampler(n)
        sid = rng.choice(sep.lens.size, size=n, p=sep_p)
        a = _assemble(tok, sep, tid, sid)
        parts.append(a)
        have += a.size
    return np.concatenate(parts)[:nbytes]


def write_dict(path: str, words: list[bytes]):
    """32-byte-aligned dictionary: one word per slot, NUL padded."""
    buf = bytearray(32 * len(words))
    for i, w in enumerate(words):
        assert 0 < len(w) <= 32
        buf[32 * i:32 * i + len(w)] = w
    with open(path, "wb") as f:
        f.write(bytes(buf))


def write_list(path: str, paths: list[str]):
    with open(path, "w") as f:
        for p in paths:
            f.write(p + "\n")


def c1_corpus(root: str | None = None, seed: int = 1, nfiles: int = 16, file_bytes: int = 512 << 10,
              nwords: int = 64) -> dict:
    """C1: 64-word dictionary, 16 x 512 KiB synthetic text."""
    root = root or os.path.join(SHM, f"gfs_c1_s{seed}_{nfiles}x{file_bytes}_{nwords}")
    params = {"kind": "c1", "seed": seed, "nfiles": nfiles, "file_bytes": file_bytes, "nwords": nwords}
    res = {"root": root, "dict": os.path.join(root, "dict.bin"), "list": os.path.join(root, "files.txt")}
    if _marker_ok(root, params):
        res["paths"] = [l.strip() for l in open(res["list"]) if l.strip()]
        return res
    shutil.rmtree(root, ignore_errors=True)
    os.makedirs(root)
    lex = lexicon(20000, seed)
    rng = np.random.default_rng(seed + 1)
    dict_idx = rng.choice(len(lex), size=nwords, replace=False)
    # bias the text so ~1-3% of tokens are dictionary words: the dictionary is
    # drawn uniformly, the text is Zipf over a shuffled lexicon.
    words = [lex[i] for i in dict_idx]
    ids = random_identifiers(2000, rng)
    vocab = lex + ids
    tok = _Vocab(vocab)
    sep = _Vocab([b" ", b"\n", b", ", b". ", b"; ", b"(", b") ", b"\t", b"-", b"\r\n", b"\xc3\xa9 ", b"'"])
    sep_p = np.array([0.55, 0.1, 0.08, 0.07, 0.03, 0.03, 0.03, 0.03, 0.02, 0.02, 0.02, 0.02])
    sep_p /= sep_p.sum()
    nlex = len(lex)

    def sampler(n):
        t = _zipf_ids(rng, nlex, n, 1.1)
        is_id = rng.random(n) < 0.10
        t[is_id] = nlex + rng.integers(0, len(ids), size=int(is_id.sum()))
        # sprinkle dictionary words (they are uniform draws, mostly rare in Zipf)
        is_d = rng.random(n) < 0.02
        t[is_d] = dict_idx[rng.integers(0, nwords, size=int(is_d.sum()))]
        return t

    paths = []
    for f in range(nfiles):
        p = os.path.join(root, f"doc{f:03d}.txt")
        text = text_stream(file_bytes, rng, tok, sampler, sep, sep_p)
        with open(p, "wb") as fh:
            fh.write(text.tobytes())
        paths.append(p)
    write_dict(res["dict"], words)
    write_list(res["list"], paths)
    _mark(root, params)
    res["paths"] = paths
    return res


_C_KEYWORDS = [b"int", b"return", b"if", b"else", b"for", b"while", b"struct", b"static", b"void",
               b"unsigned", b"long", b"char", b"const", b"sizeof", b"break", b"case", b"switch",
               b"goto", b"NULL", b"u32", b"u64", b"define", b"include", b"endif", b"ifdef"]


def c4_sizes(nfiles: int, total: int, rng) -> np.ndarray:
    s = rng.lognormal(mean=np.log(7 * 1024), sigma=1.3, size=nfiles)
    s = np.clip(s, 64, 4 << 20)
    for _ in range(8):  # rescale to the total, keeping the clip
        s = np.clip(s * (total / s.sum()), 64, 4 << 20)
    s = np.floor(s).astype(np.int64)
    s[0] += total - int(s.sum())  # exact total
    s = np.clip(s, 1, None)
    return s


def c4_corpus(root: str | None = None, seed: int = 4, nfiles: int = 30000, total_bytes: int = 500 << 20,
              nwords: int = 58000) -> dict:
    """C4: Linux-source-shaped tree with a 58k-word dictionary."""
    root = root or os.path.join(SHM, f"gfs_c4_s{seed}_{nfiles}_{total_bytes}_{nwords}")
    params = {"kind": "c4", "seed": seed, "nfiles": nfiles, "total": total_bytes, "nwords": nwords}
    res = {"root": root, "dict": os.path.join(root, "dict.bin"), "list": os.path.join(root, "files.txt")}
    if _marker_ok(root, params):
        res["paths"] = [l.strip() for l in open(res["list"]) if l.strip()]
        res["sizes"] = [os.path.getsize(p) for p in res["paths"]]
        return res
    shutil.rmtree(root, ignore_errors=True)
    os.makedirs(root)
    rng = np.random.default_rng(seed)
    lex = lexicon(int(nwords * 1.4), seed, min_len=1, max_len=28, mean=8.5)
    order = rng.permutation(len(lex))
    words = [lex[i] for i in order[:nwords]]
    compounds = []
    for _ in range(20000):
        a, b = rng.integers(0, len(lex), size=2)
        c = lex[a] + b"_" + lex[b]
        if rng.random() < 0.3:
            c += str(int(rng.integers(0, 100))).encode()
        compounds.append(c)
    numbers = [str(int(x)).encode() for x in rng.integers(0, 100000, size=2000)] + \
              [("0x%x" % int(x)).encode() for x in rng.integers(0, 1 << 20, size=1000)]
    vocab = lex + compounds + _C_KEYWORDS + numbers
    n_lex, n_cmp, n_kw, n_num = len(lex), len(compounds), len(_C_KEYWORDS), len(numbers)
    tok = _Vocab(vocab)
    seps = [b" ", b"\n", b"\t", b"(", b") ", b";\n", b" = ", b", ", b"->", b"/* ", b" */\n",
            b"\n\t", b" {\n", b"}\n", b" + ", b"*", b"[", b"]", b".", b"#", b" <", b">\n", b" && ",
            b" == ", b"\n\n", b"\t\t", b" - "]
    sep = _Vocab(seps)
    sep_p = np.array([0.30, 0.08, 0.05, 0.06, 0.06, 0.07, 0.04, 0.05, 0.03, 0.02, 0.02, 0.04,
                      0.02, 0.02, 0.01, 0.02, 0.01, 0.01, 0.03, 0.005, 0.005, 0.005, 0.01, 0.01,
                      0.03, 0.02, 0.01])
    sep_p /= sep_p.sum()

    def sampler(n):
        u = rng.random(n)
        t = _zipf_ids(rng, n_lex, n, 1.05)
        m_cmp = u < 0.25
        t[m_cmp] = n_lex + rng.integers(0, n_cmp, size=int(m_cmp.sum()))
        m_kw = (u >= 0.25) & (u < 0.40)
        t[m_kw] = n_lex + n_cmp + rng.integers(0, n_kw, size=int(m_kw.sum()))
        m_num = (u >= 0.40) & (u < 0.45)
        t[m_num] = n_lex + n_cmp + n_kw + rng.integers(0, n_num, size=int(m_num.sum()))
        return t

    sizes = c4_sizes(nfiles, total_bytes, rng)
    dirs = []
    for d in range(max(1, nfiles // 40)):
        depth = int(rng.integers(3, 6))
        parts = [lex[int(rng.integers(0, n_lex))].decode()[:12] or "d" for _ in range(depth - 1)]
        dirs.append(os.path.join(root, "src", *[f"{p}{d % 97}" for p in parts]))
    paths = []
    stream = None
    pos = 0
    chunk = 64 << 20
    for i in range(nfiles):
        sz = int(sizes[i])
        if stream is None or pos + sz > stream.size:
            need = max(chunk, sz)
            rest = stream[pos:] if stream is not None else np.zeros(0, np.uint8)
            stream = np.concatenate([rest, text_stream(need, rng, tok, sampler, sep, sep_p)])
            pos = 0
        d = dirs[i % len(dirs)]
        os.makedirs(d, exist_ok=True)
        name = lex[int(rng.integers(0, n_lex))].decode()[:20] or "f"
        p = os.path.join(d, f"{name}_{i}.{'c' if rng.random() < 0.7 else 'h'}")
        with open(p, "wb") as fh:
            fh.write(stream[pos:pos + sz].tobytes())
        pos += sz
        paths.append(p)
    write_dict(res["dict"], words)
    write_list(res["list"], paths)
    _mark(root, params)
    res["paths"] = paths
    res["sizes"] = [int(s) for s in sizes]
    return res


def tiny_corpus(root: str, seed: int, nfiles: int = 4, max_bytes: int = 3000, nwords: int = 12,
                extra_files: list[bytes] | None = None, extra_words: list[bytes] | None = None) -> dict:
    """Small random corpus for brute-force pins: small alphabet so words collide often."""
    os.makedirs(root, exist_ok=True)
    rng = np.random.default_rng(seed)
    alpha = np.frombuffer(b"ab_1 .\n", dtype=np.uint8)
    p = np.array([0.3, 0.3, 0.05, 0.05, 0.2, 0.05, 0.05])
    words = set()
    while len(words) < nwords:
        L = int(rng.integers(1, 5))
        words.add(rng.choice(alpha[:4], size=L, p=p[:4] / p[:4].sum()).tobytes())
    words = sorted(words)
    if extra_words:
        words += extra_words
    paths = []
    for f in range(nfiles):
        n = int(rng.integers(0, max_bytes))
        data = rng.choice(alpha, size=n, p=p).tobytes()
        fp = os.path.join(root, f"t{f}.txt")
        with open(fp, "wb") as fh:
            fh.write(data)
        paths.append(fp)
    for j, data in enumerate(extra_files or []):
        fp = os.path.join(root, f"x{j}.txt")
        with open(fp, "wb") as fh:
            fh.write(data)
        paths.append(fp)
    write_dict(os.path.join(root, "dict.bin"), words)
    write_list(os.path.join(root, "files.txt"), paths)
    return {"root": root, "dict": os.path.join(root, "dict.bin"), "list": os.path.join(root, "files.txt"),
            "paths": paths, "words": words}


# ----------------------------------------------------------------- C3 matrix
def matrix_files(root: str, rows: int, cols: int, seed: int = 3, integer: bool = False) -> dict:
    """Row-major little-endian fp32 A (rows x cols) and x (cols): U[0,1) or A in {0,1,2}, x in {0,1}."""
    os.makedirs(root, exist_ok=True)
    tag = f"{'int' if integer else 'u01'}_{rows}x{cols}_s{seed}"
    a_path = os.path.join(root, f"A_{tag}.f32")
    x_path = os.path.join(root, f"x_{tag}.f32")
    params = {"kind": "matrix", "rows": rows, "cols": cols, "seed": seed, "integer": integer}
    if _marker_ok(a_path, params) and os.path.exists(x_path):
        return {"A": a_path, "x": x_path, "rows": rows, "cols": cols}
    rng = np.random.default_rng(seed)
    tmp = a_path + f".tmp{os.getpid()}"
    with open(tmp, "wb") as f:
        step = max(1, (64 << 20) // (4 * cols))
        for r0 in range(0, rows, step):
            n = min(step, rows - r0)
            if integer:
                a = rng.integers(0, 3, size=(n, cols)).astype("<f4")
            else:
                a = rng.random((n, cols), dtype=np.float32).astype("<f4")
            f.write(a.tobytes())
    os.replace(tmp, a_path)
    x = rng.integers(0, 2, size=cols).astype("<f4") if integer else rng.random(cols, dtype=np.float32)
    with open(x_path, "wb") as f:
        f.write(x.astype("<f4").tobytes())
    _mark(a_path, params)
    return {"A": a_path, "x": x_path, "rows": rows, "cols": cols}


# ----------------------------------------------------------------- call lists
def random_calls(seed: int, n: int, file_size: int, max_len: int, page_size: int | None = None,
                 edge_frac: float = 0.2) -> tuple[np.ndarray, np.ndarray]:
    """(offsets, lengths) for gread parity: random spans plus edge cases
    (len 0, off == S, off > S, page-straddling, last partial page)."""
    rng = np.random.default_rng(seed)
    off = rng.integers(0, max(file_size, 1), size=n, dtype=np.int64)
    ln = rng.integers(0, max_len + 1, size=n, dtype=np.int64)
    k = int(n * edge_frac)
    if k:
        which = rng.integers(0, 6, size=k)
        for i, w in enumerate(which):
            if w == 0:
                ln[i] = 0
            elif w == 1:
                off[i] = file_size
            elif w == 2:
                off[i] = file_size + int(rng.integers(1, 1 << 20))
            elif w == 3 and page_size:
                pg = int(rng.integers(1, max(2, file_size // page_size)))
                off[i] = max(0, pg * page_size - int(rng.integers(1, 64)))
                ln[i] = int(rng.integers(64, 2 * page_size + 128))
            elif w == 4:
                off[i] = max(0, file_size - int(rng.integers(1, 4096)))
                ln[i] = int(rng.integers(1, 8192))
            else:
                ln[i] = max_len
    return off.astype(np.uint64), ln.astype(np.uint64)
