"""paper_conf_asplos_silbersteinfkw13_b200 — B200-native GPUfs buffer-cache read path.

Thin Python binding over ``libgpufs.so`` (include/gpufs.h): argument
marshalling only. Every step of the path (gopen, radix lookup, miss RPC,
eviction, hit copy, gwrite/gfsync, the consumer kernels) runs in the CUDA
library and its host daemon. PyTorch is used only for device memory and
streams. There is no CPU fallback: if the library is missing or no GPU is
present, the calls raise.
"""
from __future__ import annotations

import ctypes
import os

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libgpufs.so")

COUNTERS = ["hit", "miss", "zero_fill", "lockfree", "locked", "retry", "evict", "writeback", "rpc",
            "rpc_open", "rpc_read", "rpc_write", "bytes_h2d", "bytes_d2h", "open_fast", "reopen_valid",
            "invalidate", "enomem", "timeout", "gread_calls", "gread_bytes", "gwrite_calls", "nodes",
            "ring_wait", "busy", "stage_wait", "peer_fill", "bytes_peer", "peer_miss", "zc_fill",
            "ra_issued", "ra_adopted", "ra_reaped"]
HOST_COUNTERS = ["rpc", "read", "write", "open", "close", "trunc", "bytes_h2d", "bytes_d2h", "pread_ns",
                 "errors", "merges", "busy_ns", "open_ns", "open_sys_ns", "open_prefetch_ns", "open_table_ns",
                 "mapped_reads", "open_vt_ns"]

O_RDONLY = 0
O_GWRONCE = 1
O_RDWR = 2
PROT_WRITE = 2
F_LOCKED_TRAVERSAL = 1
FAULT_EIO = 1    # gfs_config.fault kinds (tests): a READ fails with -EIO
FAULT_SHORT = 2  # ... or comes back with half its bytes
F_NO_DMA_COMPLETION = 2
DAEMON_SPAWN = 0
DAEMON_RUN = 1


class GfsError(OSError):
    pass


class gfs_config(ctypes.Structure):
    _fields_ = [("device", ctypes.c_int), ("cache_bytes", ctypes.c_uint64), ("page_size", ctypes.c_uint32),
                ("ring_slots", ctypes.c_uint32), ("daemon_threads", ctypes.c_uint32),
                ("max_files", ctypes.c_uint32), ("max_nodes", ctypes.c_uint32), ("max_batch", ctypes.c_uint32),
                ("flags", ctypes.c_uint32), ("staging_slots", ctypes.c_uint32), ("timeout_ms", ctypes.c_uint64),
                ("frame_pool", ctypes.c_void_p), ("readahead", ctypes.c_uint32), ("fault", ctypes.c_uint32)]


class gfs_grep_params(ctypes.Structure):
    _fields_ = [("max_files", ctypes.c_uint32), ("max_words", ctypes.c_uint32), ("list_cap", ctypes.c_uint64),
                ("pair_cap", ctypes.c_uint64), ("hit_cap", ctypes.c_uint64), ("chunk", ctypes.c_uint32),
                ("grid", ctypes.c_uint32), ("block", ctypes.c_uint32), ("keep_open", ctypes.c_uint32),
                ("corpus_cap", ctypes.c_uint64), ("file_ids", ctypes.c_void_p), ("rec_cap", ctypes.c_uint64),
                ("whole_max", ctypes.c_uint32), ("scan", ctypes.c_uint32)]


class gfs_export_desc(ctypes.Structure):
    """include/gpufs.h gfs_export_desc: plain bytes describing a cache for gfs_attach_peer."""
    _fields_ = [("magic", ctypes.c_uint64), ("pid", ctypes.c_int32), ("device", ctypes.c_int32),
                ("page_shift", ctypes.c_uint32), ("nframes", ctypes.c_uint32), ("max_nodes", ctypes.c_uint32),
                ("max_files", ctypes.c_uint32), ("ptr", ctypes.c_uint64 * 7), ("ipc", (ctypes.c_ubyte * 64) * 7)]


GREP_SUMMARY = ["nrecords", "nhits", "digest_sum", "digest_xor", "nfiles", "nwords", "bytes", "err",
                "nhits_listed", "nitems"]

_lib = None


def lib():
    """Load libgpufs.so (built in-tree by build.py / __graft_entry__.build())."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} is missing: run `python -m paper_conf_asplos_silbersteinfkw13_b200.build`"
                              " (there is no CPU fallback)")
        L = ctypes.CDLL(LIB_PATH)
        P, I, U32, U64 = ctypes.c_void_p, ctypes.c_int, ctypes.c_uint32, ctypes.c_uint64
        CS = ctypes.c_char_p
        sig = {
            "gfs_config_default": ([ctypes.POINTER(gfs_config)], I),
            "gfs_init": ([ctypes.POINTER(gfs_config), ctypes.POINTER(P)], I),
            "gfs_daemon": ([P, I], I),
            "gfs_daemon_stop": ([P], I),
            "gfs_shutdown": ([P], I),
            "gfs_device_ctx": ([P], P),
            "gfs_stats": ([P, P, I, I], I),
            "gfs_host_stats": ([P, P, I], I),
            "gfs_info": ([P, P, I], I),
            "gfs_export": ([P, ctypes.POINTER(gfs_export_desc)], I),
            "gfs_register_file": ([P, CS], I),
            "gfs_attach_peer": ([P, ctypes.POINTER(gfs_export_desc)], I),
            "gfs_run_gread": ([P, P, CS, I, U32, P, P, P, P, P, U32, U32, U32], I),
            "gfs_run_seqread": ([P, P, CS, U64, U64, U64, I, P, P, P, U32, U32], I),
            "gfs_run_randread": ([P, P, CS, I, P, U32, U32, P, P, P, U32, U32], I),
            "gfs_probe_h2d": ([P, U64, U32, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ctypes.c_double)], I),
            "gfs_run_randread_warp": ([P, P, CS, I, P, U32, U32, P, P, P, U32, U32], I),
            "gfs_run_randread_async": ([P, P, CS, I, P, U32, U32, U32, P, P, P, U32, U32], I),
            "gfs_run_gwrite": ([P, P, CS, U32, P, P, P, P, P, U32, U32, I], I),
            "gfs_run_mmap_write": ([P, P, CS, U32, P, P, P, P, P, U32, U32, I], I),
            "gfs_run_fileop": ([P, P, CS, I, I, U64, P], I),
            "gfs_run_seqwrite": ([P, P, CS, U64, U64, P, P, P, U32, U32, U32], I),
            "gfs_grep_work_bytes": ([ctypes.POINTER(gfs_grep_params)], U64),
            "gfs_grep": ([P, P, CS, CS, ctypes.POINTER(gfs_grep_params), P, P, U64, P, P, P], I),
            "gfs_grep_graph_create": ([P, P, CS, CS, ctypes.POINTER(gfs_grep_params), P, P, U64, P, P, P,
                                       ctypes.POINTER(P)], I),
            "gfs_grep_graph_launch": ([P, P], I),
            "gfs_grep_graph_destroy": ([P], I),
            "gfs_matvec": ([P, P, CS, CS, CS, U64, U64, P, P, P, U32, U32], I),
            "gfs_matvec_rows": ([P, P, CS, CS, CS, U64, U64, U64, U64, P, P, P, U32, U32], I),
        }
        for name, (args, res) in sig.items():
            fn = getattr(L, name)
            fn.argtypes = args
            fn.restype = res
        _lib = L
    return _lib


def _ck(r: int, what: str) -> int:
    if r < 0:
        raise GfsError(-r, f"{what}: {os.strerror(-r)}")
    return r


def _b(path) -> bytes:
    return os.fsencode(path)


# ------------------------------------------------------------------ host API
def gfs_config_default(**kw) -> gfs_config:
    c = gfs_config()
    _ck(lib().gfs_config_default(ctypes.byref(c)), "gfs_config_default")
    for k, v in kw.items():
        setattr(c, k, v)
    return c


def gfs_init(cfg: gfs_config) -> int:
    h = ctypes.c_void_p()
    _ck(lib().gfs_init(ctypes.byref(cfg), ctypes.byref(h)), "gfs_init")
    return h.value


def gfs_daemon(h: int, mode: int = DAEMON_SPAWN) -> int:
    return _ck(lib().gfs_daemon(h, mode), "gfs_daemon")


def gfs_daemon_stop(h: int) -> int:
    return _ck(lib().gfs_daemon_stop(h), "gfs_daemon_stop")


def gfs_shutdown(h: int) -> int:
    return _ck(lib().gfs_shutdown(h), "gfs_shutdown")


def gfs_device_ctx(h: int) -> int:
    return lib().gfs_device_ctx(h)


def gfs_stats(h: int, reset: bool = False) -> dict:
    a = (ctypes.c_uint64 * len(COUNTERS))()
    _ck(lib().gfs_stats(h, a, len(COUNTERS), 1 if reset else 0), "gfs_stats")
    return dict(zip(COUNTERS, (int(x) for x in a)))


def gfs_host_stats(h: int) -> dict:
    a = (ctypes.c_uint64 * len(HOST_COUNTERS))()
    _ck(lib().gfs_host_stats(h, a, len(HOST_COUNTERS)), "gfs_host_stats")
    return dict(zip(HOST_COUNTERS, (int(x) for x in a)))


def gfs_info(h: int) -> dict:
    a = (ctypes.c_uint64 * 9)()
    _ck(lib().gfs_info(h, a, 9), "gfs_info")
    return dict(zip(["page_size", "nframes", "max_files", "max_nodes", "ring_slots", "daemon_threads",
                     "staging_slots", "host_next_ticket", "device_ring_tail"], (int(x) for x in a)))


def gfs_register_file(h: int, path) -> int:
    """Zero-copy misses for `path` (include/gpufs.h gfs_register_file)."""
    return _ck(lib().gfs_register_file(h, _b(path)), "gfs_register_file")


def gfs_export(h: int) -> bytes:
    """Describe cache h for gfs_attach_peer (in this or another process)."""
    d = gfs_export_desc()
    _ck(lib().gfs_export(h, ctypes.byref(d)), "gfs_export")
    return bytes(d)


def gfs_attach_peer(h: int, desc: bytes) -> int:
    """Attach the cache described by `desc` (gfs_export) as a peer of h; returns its index."""
    d = gfs_export_desc.from_buffer_copy(desc)
    return _ck(lib().gfs_attach_peer(h, ctypes.byref(d)), "gfs_attach_peer")


# ------------------------------------------------------------------ launchers
def gfs_run_gread(h, stream, path, mode, ncalls, d_off, d_len, d_dstoff, d_dst, d_ret, grid, block, smem=0):
    return _ck(lib().gfs_run_gread(h, stream, _b(path), mode, ncalls, d_off, d_len, d_dstoff, d_dst, d_ret,
                                   grid, block, smem), "gfs_run_gread")


def gfs_run_seqread(h, stream, path, file_off, total, chunk, use_mmap, d_scratch, d_sum, d_err, grid, block):
    return _ck(lib().gfs_run_seqread(h, stream, _b(path), file_off, total, chunk, use_mmap, d_scratch, d_sum,
                                     d_err, grid, block), "gfs_run_seqread")


def gfs_probe_h2d(stream, nbytes=256 << 20, reps=10):
    """(copy-engine GB/s, SM-pull GB/s) of the host->device link (include/gpufs.h)."""
    ce, sm = ctypes.c_double(0), ctypes.c_double(0)
    _ck(lib().gfs_probe_h2d(stream, nbytes, reps, ctypes.byref(ce), ctypes.byref(sm)), "gfs_probe_h2d")
    return ce.value, sm.value


def gfs_run_randread(h, stream, path, raw, d_raw, chunk, calls_per_block, d_off, d_sum, d_err, grid, block):
    return _ck(lib().gfs_run_randread(h, stream, _b(path) if path else None, raw, d_raw, chunk, calls_per_block,
                                      d_off, d_sum, d_err, grid, block), "gfs_run_randread")


def gfs_run_randread_async(h, stream, path, raw, d_raw, chunk, calls_per_block, depth, d_off, d_sum, d_err, grid,
                           block):
    return _ck(lib().gfs_run_randread_async(h, stream, _b(path) if path else None, raw, d_raw, chunk, calls_per_block,
                                            depth, d_off, d_sum, d_err, grid, block), "gfs_run_randread_async")


def gfs_run_randread_warp(h, stream, path, raw, d_raw, chunk, calls_per_block, d_off, d_sum, d_err, grid, block):
    return _ck(lib().gfs_run_randread_warp(h, stream, _b(path) if path else None, raw, d_raw, chunk,
                                           calls_per_block, d_off, d_sum, d_err, grid, block),
               "gfs_run_randread_warp")


def gfs_run_seqwrite(h, stream, path, total, chunk, d_src, d_err, d_tmp, grid, block, sync_grid):
    return _ck(lib().gfs_run_seqwrite(h, stream, _b(path), total, chunk, d_src, d_err, d_tmp, grid, block,
                                      sync_grid), "gfs_run_seqwrite")


def gfs_run_gwrite(h, stream, path, ncalls, d_off, d_len, d_srcoff, d_src, d_ret, grid, block, flags=1):
    return _ck(lib().gfs_run_gwrite(h, stream, _b(path), ncalls, d_off, d_len, d_srcoff, d_src, d_ret, grid,
                                    block, flags), "gfs_run_gwrite")


def gfs_run_mmap_write(h, stream, path, ncalls, d_off, d_len, d_srcoff, d_src, d_ret, grid, block, do_msync):
    return _ck(lib().gfs_run_mmap_write(h, stream, _b(path), ncalls, d_off, d_len, d_srcoff, d_src, d_ret, grid,
                                        block, do_msync), "gfs_run_mmap_write")


def gfs_run_fileop(h, stream, path, flags, op, arg, d_ret):
    return _ck(lib().gfs_run_fileop(h, stream, _b(path), flags, op, arg, d_ret), "gfs_run_fileop")


def gfs_grep_work_bytes(p: gfs_grep_params) -> int:
    return int(lib().gfs_grep_work_bytes(ctypes.byref(p)))


def gfs_grep(h, stream, dict_path, list_path, p: gfs_grep_params, d_work, d_rec, rec_cap, d_totals, d_hits,
             d_summary):
    return _ck(lib().gfs_grep(h, stream, _b(dict_path), _b(list_path), ctypes.byref(p), d_work, d_rec, rec_cap,
                              d_totals, d_hits, d_summary), "gfs_grep")


def gfs_grep_graph_create(h, stream, dict_path, list_path, p: gfs_grep_params, d_work, d_rec, rec_cap, d_totals,
                          d_hits, d_summary):
    g = ctypes.c_void_p()
    _ck(lib().gfs_grep_graph_create(h, stream, _b(dict_path), _b(list_path), ctypes.byref(p), d_work, d_rec,
                                    rec_cap, d_totals, d_hits, d_summary, ctypes.byref(g)), "gfs_grep_graph_create")
    return g


def gfs_grep_graph_launch(g, stream):
    return _ck(lib().gfs_grep_graph_launch(g, stream), "gfs_grep_graph_launch")


def gfs_grep_graph_destroy(g):
    return _ck(lib().gfs_grep_graph_destroy(g), "gfs_grep_graph_destroy")


def gfs_matvec(h, stream, a_path, x_path, y_path, rows, cols, d_x, d_y, d_err, grid, block):
    return _ck(lib().gfs_matvec(h, stream, _b(a_path), _b(x_path), _b(y_path), rows, cols, d_x, d_y, d_err, grid,
                                block), "gfs_matvec")


def gfs_matvec_rows(h, stream, a_path, x_path, y_path, rows, cols, row0, nrows, d_x, d_y, d_err, grid, block):
    return _ck(lib().gfs_matvec_rows(h, stream, _b(a_path), _b(x_path), _b(y_path), rows, cols, row0, nrows, d_x,
                                     d_y, d_err, grid, block), "gfs_matvec_rows")


from . import build  # noqa: E402,F401
from .api import GpuFS  # noqa: E402  (torch-facing convenience wrapper)
