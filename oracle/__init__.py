"""CPU oracle for the GPUfs buffer-cache read path — TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline``
leg (and ``bench.py --impl reference``) may import this package. The product
package ``paper_conf_asplos_silbersteinfkw13_b200`` never imports it and shares
no code with it.

The oracle itself is ``oracle.cpp`` (C++17 over POSIX pread/pwrite); this module
only builds it with g++ and marshals arguments through ctypes. Every oracle
function cites the PAPER.md passage it writes out (see oracle.cpp).
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.cpp")
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.cpp -> liboracle.so (g++ -O2). Building the checker is not using it."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["g++", "-O2", "-std=c++17", "-shared", "-fPIC", "-pthread",
                               "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


def lib():
    global _lib
    with _lock:
        if _lib is None:
            build()
            L = ctypes.CDLL(_LIB)
            u64, i64, p = ctypes.c_uint64, ctypes.c_int64, ctypes.c_void_p
            cs, ci = ctypes.c_char_p, ctypes.c_int
            L.orc_pread.argtypes = [cs, u64, u64, u64, p]; L.orc_pread.restype = i64
            L.orc_file_size.argtypes = [cs]; L.orc_file_size.restype = i64
            L.orc_checksum.argtypes = [cs, u64, u64, ctypes.POINTER(u64)]; L.orc_checksum.restype = i64
            L.orc_checksum_mt.argtypes = [cs, u64, u64, ci, ctypes.POINTER(u64)]; L.orc_checksum_mt.restype = i64
            L.orc_checksum_calls.argtypes = [cs, p, u64, u64, ci, ctypes.POINTER(u64)]
            L.orc_checksum_calls.restype = i64
            L.orc_cache_new.argtypes = [u64, u64]; L.orc_cache_new.restype = p
            L.orc_cache_free.argtypes = [p]; L.orc_cache_free.restype = None
            L.orc_cache_open.argtypes = [p, cs, ci]; L.orc_cache_open.restype = ci
            L.orc_cache_close.argtypes = [p, ci]; L.orc_cache_close.restype = ci
            L.orc_cache_size.argtypes = [p, ci]; L.orc_cache_size.restype = i64
            L.orc_cache_read.argtypes = [p, ci, u64, u64, p]; L.orc_cache_read.restype = i64
            L.orc_cache_mmap_copy.argtypes = [p, ci, u64, u64, p]; L.orc_cache_mmap_copy.restype = i64
            L.orc_cache_write.argtypes = [p, ci, u64, u64, p]; L.orc_cache_write.restype = i64
            L.orc_cache_mmap_write.argtypes = [p, ci, u64, u64, p, ci]; L.orc_cache_mmap_write.restype = i64
            L.orc_cache_fsync.argtypes = [p, ci]; L.orc_cache_fsync.restype = ci
            L.orc_cache_ftruncate.argtypes = [p, ci, u64]; L.orc_cache_ftruncate.restype = ci
            L.orc_cache_stats.argtypes = [p, p]; L.orc_cache_stats.restype = None
            L.orc_grep.argtypes = [cs, cs, ci, ci, ctypes.POINTER(p)]; L.orc_grep.restype = ci
            L.orc_grep_brute.argtypes = [cs, cs, ctypes.POINTER(p)]; L.orc_grep_brute.restype = ci
            L.orc_grep_counts.argtypes = [p, p]; L.orc_grep_counts.restype = None
            L.orc_grep_get.argtypes = [p] + [p] * 8; L.orc_grep_get.restype = None
            L.orc_grep_free.argtypes = [p]; L.orc_grep_free.restype = None
            L.orc_matvec.argtypes = [cs, cs, u64, u64, u64, u64, ci, p]; L.orc_matvec.restype = ci
            _lib = L
    return _lib


def _b(s) -> bytes:
    return os.fsencode(s)


def _ptr(a: np.ndarray):
    return ctypes.c_void_p(a.ctypes.data)


class OracleError(OSError):
    pass


def _check(r):
    if r < 0:
        raise OracleError(-r, os.strerror(-r))
    return r


# ---------------------------------------------------------------- O1: gread
def pread(path, snap_size: int, off: int, length: int) -> bytes:
    """gread's plain definition: pread of [off, off+min(len, S-off))."""
    out = np.zeros(max(length, 1), dtype=np.uint8)
    n = _check(lib().orc_pread(_b(path), snap_size, off, length, _ptr(out)))
    return out[:n].tobytes()


def file_size(path) -> int:
    return _check(lib().orc_file_size(_b(path)))


def checksum(path, off: int, length: int) -> int:
    """Position-weighted u64 checksum of file bytes [off, off+len) (R9)."""
    s = ctypes.c_uint64(0)
    _check(lib().orc_checksum(_b(path), off, length, ctypes.byref(s)))
    return s.value


def checksum_mt(path, off: int, length: int, nthreads: int = 0) -> int:
    """The same checksum of [off, off+len), the range cut into nthreads pieces
    (the sum is per byte, so pieces add up mod 2^64). nthreads 0: os.cpu_count()."""
    s = ctypes.c_uint64(0)
    _check(lib().orc_checksum_mt(_b(path), off, length, nthreads or os.cpu_count() or 1, ctypes.byref(s)))
    return s.value


def checksum_calls(path, offs, length: int, nthreads: int = 0) -> int:
    """K4 consumer total: sum over calls i of checksum(path, offs[i], length) mod 2^64."""
    o = np.ascontiguousarray(np.asarray(offs, dtype=np.uint64))
    s = ctypes.c_uint64(0)
    _check(lib().orc_checksum_calls(_b(path), _ptr(o) if o.size else None, o.size, length,
                                    nthreads or os.cpu_count() or 1, ctypes.byref(s)))
    return s.value


class PageCache:
    """Page-cache model of P:L587-622 (O1/O2). flags: 0 = O_RDONLY, 1 = O_GWRONCE,
    2 = O_RDWR (pristine copy + diff write-back)."""

    RDONLY = 0
    GWRONCE = 1
    RDWR = 2

    def __init__(self, page_size: int, capacity_pages: int):
        self.h = lib().orc_cache_new(page_size, capacity_pages)
        if not self.h:
            raise ValueError("bad page cache geometry")
        self.P = page_size

    def close_all(self):
        if self.h:
            lib().orc_cache_free(self.h)
            self.h = None

    __del__ = close_all

    def open(self, path, flags=0) -> int:
        return _check(lib().orc_cache_open(self.h, _b(path), flags))

    def close(self, fd):
        return _check(lib().orc_cache_close(self.h, fd))

    def size(self, fd) -> int:
        return _check(lib().orc_cache_size(self.h, fd))

    def read(self, fd, off, length) -> bytes:
        out = np.zeros(max(length, 1), dtype=np.uint8)
        n = _check(lib().orc_cache_read(self.h, fd, off, length, _ptr(out)))
        return out[:n].tobytes()

    def mmap_copy(self, fd, off, length) -> bytes:
        out = np.zeros(max(length, 1), dtype=np.uint8)
        n = _check(lib().orc_cache_mmap_copy(self.h, fd, off, length, _ptr(out)))
        return out[:n].tobytes()

    def write(self, fd, off, data) -> int:
        a = np.frombuffer(bytes(data), dtype=np.uint8).copy()
        return _check(lib().orc_cache_write(self.h, fd, off, len(a), _ptr(a) if len(a) else None))

    def mmap_write(self, fd, off, data, msync=False) -> int:
        """Writable gmmap of an O_RDWR file + stores (+ gmsync); returns the mapped prefix length."""
        a = np.frombuffer(bytes(data), dtype=np.uint8).copy()
        return _check(lib().orc_cache_mmap_write(self.h, fd, off, len(a), _ptr(a) if len(a) else None,
                                                 1 if msync else 0))

    def fsync(self, fd):
        return _check(lib().orc_cache_fsync(self.h, fd))

    def ftruncate(self, fd, size):
        return _check(lib().orc_cache_ftruncate(self.h, fd, size))

    def stats(self) -> dict:
        a = np.zeros(5, dtype=np.uint64)
        lib().orc_cache_stats(self.h, _ptr(a))
        return dict(zip(["hits", "misses", "evictions", "writebacks", "resident"], map(int, a)))


# ---------------------------------------------------------------- O3: grep -w
class GrepResult:
    def __init__(self, rec_f, rec_k, rec_c, totals, digest, hits, nbytes, nfiles):
        self.rec_f, self.rec_k, self.rec_c = rec_f, rec_k, rec_c
        self.totals, self.digest, self.hits = totals, digest, hits
        self.bytes, self.nfiles = nbytes, nfiles

    @property
    def records(self) -> np.ndarray:
        """(n,3) uint64 array of (file, word, count), sorted by (file, word)."""
        return np.stack([self.rec_f.astype(np.uint64), self.rec_k.astype(np.uint64),
                         self.rec_c.astype(np.uint64)], axis=1) if len(self.rec_f) else \
            np.zeros((0, 3), dtype=np.uint64)


def _grep_collect(h, want_hits=True) -> GrepResult:
    L = lib()
    c = np.zeros(6, dtype=np.uint64)
    L.orc_grep_counts(h, _ptr(c))
    nrec, nw, nh, nlist, nbytes, nfiles = map(int, c)
    rf = np.zeros(max(nrec, 1), np.uint32); rk = np.zeros(max(nrec, 1), np.uint32)
    rc = np.zeros(max(nrec, 1), np.uint64); tot = np.zeros(max(nw, 1), np.uint64)
    dg = np.zeros(2, np.uint64)
    hf = np.zeros(max(nlist, 1), np.uint32); ho = np.zeros(max(nlist, 1), np.uint64)
    hk = np.zeros(max(nlist, 1), np.uint32)
    L.orc_grep_get(h, _ptr(rf), _ptr(rk), _ptr(rc), _ptr(tot), _ptr(dg), _ptr(hf), _ptr(ho), _ptr(hk))
    L.orc_grep_free(h)
    hits = np.stack([hf[:nlist].astype(np.uint64), ho[:nlist], hk[:nlist].astype(np.uint64)], axis=1) \
        if want_hits else None
    return GrepResult(rf[:nrec], rk[:nrec], rc[:nrec], tot[:nw], (int(dg[0]), int(dg[1]), nh), hits,
                      nbytes, nfiles)


def grep(dict_path, list_path, want_hits=True, nthreads=1) -> GrepResult:
    """Tokenising grep -w oracle."""
    h = ctypes.c_void_p()
    _check(lib().orc_grep(_b(dict_path), _b(list_path), 1 if want_hits else 0, nthreads, ctypes.byref(h)))
    return _grep_collect(h, want_hits)


def grep_brute(dict_path, list_path) -> GrepResult:
    """Brute-force literal grep -w definition (pin for ``grep``)."""
    h = ctypes.c_void_p()
    _check(lib().orc_grep_brute(_b(dict_path), _b(list_path), ctypes.byref(h)))
    return _grep_collect(h, True)


# ---------------------------------------------------------------- O4: matvec
def matvec(a_path, x_path, rows, cols, row0=0, nrows=None, nthreads=1) -> np.ndarray:
    """float64 y = A x."""
    nrows = rows - row0 if nrows is None else nrows
    y = np.zeros(max(nrows, 1), dtype=np.float64)
    _check(lib().orc_matvec(_b(a_path), _b(x_path), rows, cols, row0, nrows, nthreads, _ptr(y)))
    return y[:nrows]
