"""Torch-facing convenience wrapper over the C ABI (marshalling only).

torch supplies device memory and the CUDA stream; every operation is one
launcher of libgpufs.so. Methods synchronise the stream before returning
results unless ``sync=False``.
"""
from __future__ import annotations

import numpy as np

from . import (DAEMON_SPAWN, gfs_attach_peer, gfs_export, gfs_config_default, gfs_daemon, gfs_daemon_stop, gfs_host_stats, gfs_info,
               gfs_init, gfs_run_fileop, gfs_run_gread, gfs_run_gwrite, gfs_run_randread, gfs_run_seqread,
               gfs_shutdown, gfs_stats, gfs_device_ctx)


def _torch():
    import torch
    if not torch.cuda.is_available():
        raise RuntimeError("GpuFS needs a CUDA device (there is no CPU fallback)")
    return torch


class GpuFS:
    """One GPU buffer cache + its host daemon (gfs_init + gfs_daemon)."""

    def __init__(self, cache_bytes=1 << 30, page_size=64 << 10, device=0, daemon_threads=8, ring_slots=4096,
                 max_files=4096, max_nodes=0, max_batch=32, flags=0, timeout_ms=60000, staging_slots=0,
                 readahead=0, fault=0):
        torch = _torch()
        torch.cuda.set_device(device)
        self.device = device
        self.page_size = page_size
        cfg = gfs_config_default(device=device, cache_bytes=cache_bytes, page_size=page_size,
                                 daemon_threads=daemon_threads, ring_slots=ring_slots, max_files=max_files,
                                 max_nodes=max_nodes, max_batch=max_batch, flags=flags, timeout_ms=timeout_ms,
                                 staging_slots=staging_slots, readahead=readahead, fault=fault)
        self.h = gfs_init(cfg)
        gfs_daemon(self.h, DAEMON_SPAWN)

    # lifecycle --------------------------------------------------------------
    def close(self):
        if getattr(self, "h", None):
            _torch().cuda.synchronize(self.device)
            gfs_shutdown(self.h)
            self.h = None

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    def stop_daemon(self):
        gfs_daemon_stop(self.h)

    def start_daemon(self):
        gfs_daemon(self.h, DAEMON_SPAWN)

    def stats(self, reset=False) -> dict:
        return gfs_stats(self.h, reset)

    def host_stats(self) -> dict:
        return gfs_host_stats(self.h)

    def info(self) -> dict:
        return gfs_info(self.h)

    def register_file(self, path) -> int:
        """Map `path` for zero-copy misses (gfs_register_file): O_RDONLY misses of it
        are pulled straight from the host page cache, without RPCs."""
        from . import gfs_register_file
        return gfs_register_file(self.h, path)

    # peer caches (NEXT-1) -------------------------------------------------
    def export(self) -> bytes:
        """Describe this cache for attach_peer in another process or GpuFS (gfs_export)."""
        return gfs_export(self.h)

    def attach_peer(self, desc: bytes) -> int:
        """Map another cache (its export()) as a read-only peer: misses of read-only
        files are filled from it over NVLink when it holds the same version (gfs_attach_peer)."""
        return gfs_attach_peer(self.h, desc)

    @property
    def ctx(self) -> int:
        return gfs_device_ctx(self.h)

    # helpers ----------------------------------------------------------------
    def _stream(self, stream=None):
        torch = _torch()
        s = stream if stream is not None else torch.cuda.current_stream(self.device)
        return s, s.cuda_stream

    def _dev(self, a, dtype=None):
        torch = _torch()
        return torch.as_tensor(np.ascontiguousarray(a), device=f"cuda:{self.device}", dtype=dtype)

    # gread / gmmap parity harness -------------------------------------------
    def gread_calls(self, path, offs, lens, mode=0, grid=None, block=256, smem=0, stream=None, open_flags=0):
        """Issue gread (mode 0), gmmap (1), gread-to-shared (2), gread-to-shared co-aligned with the
        offset (3), warp-collective gread_warp to global (4) or to per-warp shared (5) calls;
        returns (ret, dst, dstoff)."""
        torch = _torch()
        offs = np.asarray(offs, dtype=np.uint64)
        lens = np.asarray(lens, dtype=np.uint64)
        n = len(offs)
        dstoff = np.concatenate([[0], np.cumsum(lens)[:-1]]).astype(np.uint64) if n else np.zeros(0, np.uint64)
        total = int(lens.sum()) if n else 0
        d_off = self._dev(offs.view(np.int64))
        d_len = self._dev(lens.view(np.int64))
        d_dstoff = self._dev(dstoff.view(np.int64))
        d_dst = torch.zeros(max(total, 1), dtype=torch.uint8, device=f"cuda:{self.device}")
        d_ret = torch.full((max(n, 1),), -999, dtype=torch.int64, device=f"cuda:{self.device}")
        s, sp = self._stream(stream)
        grid = grid or max(1, min(n, 296))
        if mode in (2, 3, 5) and smem == 0:
            smem = int(lens.max()) if n else 16
            smem = (smem + 15) // 16 * 16
        gfs_run_gread(self.h, sp, path, mode | (open_flags << 8), n, d_off.data_ptr(), d_len.data_ptr(), d_dstoff.data_ptr(),
                      d_dst.data_ptr(), d_ret.data_ptr(), grid, block, smem)
        s.synchronize()
        return d_ret[:n].cpu().numpy(), d_dst.cpu().numpy(), dstoff

    # sequential sweep (C2 / K1) ---------------------------------------------
    def seqread(self, path, total, chunk, file_off=0, use_mmap=False, grid=296, block=256, stream=None,
                sync=True, scratch=None, out=None, to_global=False):
        """Sequential sweep of [file_off, file_off + total) in chunk-byte calls; returns (checksum, err).
        to_global: gread only, into `scratch` (>= total bytes) at each call's file offset."""
        torch = _torch()
        dev = f"cuda:{self.device}"
        mode = 2 if to_global else (1 if use_mmap else 0)
        if scratch is None:
            n = total if to_global else (grid * chunk if not use_mmap else 1)
            scratch = torch.empty(max(1, n), dtype=torch.uint8, device=dev)
        if out is None:
            out = torch.zeros(2, dtype=torch.int64, device=dev)  # [sum, err]
        s, sp = self._stream(stream)
        gfs_run_seqread(self.h, sp, path, file_off, total, chunk, mode, scratch.data_ptr(),
                        out.data_ptr(), out.data_ptr() + 8, grid, block)
        if not sync:
            return out
        s.synchronize()
        v = out.cpu().numpy()
        return int(v[0].astype(np.uint64)), int(v[1])

    # sequential gwrite + gfsync (C5 write side) --------------------------------
    def seqwrite(self, path, src, chunk, grid=148, block=256, sync_grid=1, stream=None, sync=True, out=None):
        """gwrite the device tensor `src` (uint8) to `path` (O_GWRONCE) from `grid`
        blocks in `chunk`-byte calls, then gfsync it from `sync_grid` blocks."""
        torch = _torch()
        from . import gfs_run_seqwrite
        if out is None:
            out = torch.zeros(2, dtype=torch.int64, device=f"cuda:{self.device}")  # [err, pinned fd]
        else:
            out.zero_()
        s, sp = self._stream(stream)
        gfs_run_seqwrite(self.h, sp, path, src.numel(), chunk, src.data_ptr(), out.data_ptr(), out.data_ptr() + 8,
                         grid, block, sync_grid)
        if not sync:
            return out
        s.synchronize()
        return int(out[0].item())

    # cache-hit reads into shared memory (K4) ---------------------------------
    def randread(self, path, chunk, offs, grid, block=256, raw=None, stream=None, sync=True, out=None, warp=False,
                 depth=0, hint=False):
        """K4 reads into shared memory; warp: the warp-collective calls; depth > 0: the split-phase
        lane-parallel calls, `depth` of them in flight per block (gfs_run_randread_async); hint: every
        call names the block's next offset (gread_hint: the next lookup overlaps this copy)."""
        torch = _torch()
        dev = f"cuda:{self.device}"
        if isinstance(offs, torch.Tensor):
            d_off = offs
        else:
            d_off = self._dev(np.asarray(offs, dtype=np.uint64).view(np.int64))
        assert d_off.numel() % grid == 0
        calls = d_off.numel() // grid
        if out is None:
            out = torch.zeros(2, dtype=torch.int64, device=dev)
        s, sp = self._stream(stream)
        from . import gfs_run_randread_async, gfs_run_randread_warp
        if depth:
            gfs_run_randread_async(self.h, sp, path, 1 if raw is not None else 0,
                                   raw.data_ptr() if raw is not None else None, chunk, calls, depth,
                                   d_off.data_ptr(), out.data_ptr(), out.data_ptr() + 8, grid, block)
            if not sync:
                return out
            s.synchronize()
            v = out.cpu().numpy()
            return int(v[0].astype(np.uint64)), int(v[1])
        fn = gfs_run_randread_warp if warp else gfs_run_randread
        fn(self.h, sp, path, 1 if raw is not None else (2 if hint and not warp else 0),
                         raw.data_ptr() if raw is not None else None, chunk, calls, d_off.data_ptr(),
                         out.data_ptr(), out.data_ptr() + 8, grid, block)
        if not sync:
            return out
        s.synchronize()
        v = out.cpu().numpy()
        return int(v[0].astype(np.uint64)), int(v[1])

    # gwrite -----------------------------------------------------------------
    def gwrite_calls(self, path, offs, lens, data: bytes, srcoff=None, grid=None, block=256, stream=None,
                     flags=1, mmap=False, msync=True):
        """gwrite harness (flags: O_GWRONCE = 1 or O_RDWR = 2). mmap=True instead writes
        through gmmap(GFS_PROT_WRITE) pointers of an O_RDWR file (+ gmsync if msync)."""
        torch = _torch()
        offs = np.asarray(offs, dtype=np.uint64)
        lens = np.asarray(lens, dtype=np.uint64)
        n = len(offs)
        if srcoff is None:
            srcoff = np.concatenate([[0], np.cumsum(lens)[:-1]]).astype(np.uint64) if n else np.zeros(0, np.uint64)
        if hasattr(data, "data_ptr"):  # a device uint8 tensor already resident (no upload)
            d_src = data
        else:
            src = np.frombuffer(bytes(data), dtype=np.uint8) if len(data) else np.zeros(1, np.uint8)
            d_src = self._dev(src)
        d_off = self._dev(offs.view(np.int64))
        d_len = self._dev(lens.view(np.int64))
        d_srcoff = self._dev(np.asarray(srcoff, np.uint64).view(np.int64))
        d_ret = torch.full((max(n, 1),), -999, dtype=torch.int64, device=f"cuda:{self.device}")
        s, sp = self._stream(stream)
        if mmap:
            from . import gfs_run_mmap_write
            gfs_run_mmap_write(self.h, sp, path, n, d_off.data_ptr(), d_len.data_ptr(), d_srcoff.data_ptr(),
                               d_src.data_ptr(), d_ret.data_ptr(), grid or max(1, min(n, 296)), block,
                               1 if msync else 0)
        else:
            gfs_run_gwrite(self.h, sp, path, n, d_off.data_ptr(), d_len.data_ptr(), d_srcoff.data_ptr(),
                           d_src.data_ptr(), d_ret.data_ptr(), grid or max(1, min(n, 296)), block, flags)
        s.synchronize()
        return d_ret[:n].cpu().numpy()

    def fileop(self, path, op, flags=0, arg=0, stream=None) -> int:
        """op: 'fsync' | 'ftruncate' | 'fstat' | 'openclose'."""
        torch = _torch()
        code = {"fsync": 0, "ftruncate": 1, "fstat": 2, "openclose": 3, "pin": 4, "unpin": 5, "fsync_grid": 6}[op]
        d_ret = torch.full((1,), -999, dtype=torch.int64, device=f"cuda:{self.device}")
        s, sp = self._stream(stream)
        gfs_run_fileop(self.h, sp, path, flags, code, arg, d_ret.data_ptr())
        s.synchronize()
        return int(d_ret.item())

    # grep -w ------------------------------------------------------------------
    def grep_state(self, dict_path, list_path, hits=False, chunk=16384, grid=None, block=128, keep_open=False,
                   pair_cap=1 << 23, hit_cap=None, corpus_cap=1 << 34, rec_cap=1 << 22, file_ids=None,
                   whole_max=0, scan=0):
        """Device buffers of one grep configuration (allocated once, reused by grep(state=...)).
        Capacities come from file metadata (stat), never from file contents. file_ids: optional
        per-list-line ids reported instead of the line index (e.g. a shard's global file indices).
        whole_max: files of more than one chunk and at most this many bytes are scanned whole by
        one block (0: what the block's count table holds, 64 bytes per slot; <= chunk: every
        multi-chunk file is split). scan: 0 block scan, 1 warp scan (include/gpufs.h)."""
        import os
        torch = _torch()
        from . import gfs_grep_params, gfs_grep_work_bytes
        dev = f"cuda:{self.device}"
        nwords = max(1, os.path.getsize(dict_path) // 32)
        lbytes = os.path.getsize(list_path)
        p = gfs_grep_params(max_files=max(1, lbytes // 2 + 1), max_words=nwords, list_cap=max(lbytes, 1),
                            pair_cap=pair_cap, hit_cap=0, chunk=chunk, grid=grid or 1 << 20, block=block,
                            keep_open=1 if keep_open else 0, corpus_cap=corpus_cap, rec_cap=rec_cap,
                            whole_max=whole_max, scan=scan)
        d_ids = None
        if file_ids is not None:
            d_ids = torch.as_tensor(np.ascontiguousarray(np.asarray(file_ids, dtype=np.uint32)).view(np.int32),
                                    device=dev)
            p.file_ids = d_ids.data_ptr()
        if hits:
            p.hit_cap = hit_cap if hit_cap is not None else 1 << 22
        work = torch.empty(gfs_grep_work_bytes(p), dtype=torch.uint8, device=dev)
        rec = torch.empty(3 * rec_cap, dtype=torch.int32, device=dev)
        totals = torch.empty(nwords, dtype=torch.int64, device=dev)
        d_hits = torch.empty(2 * max(p.hit_cap, 1), dtype=torch.int64, device=dev) if hits else None
        summ = torch.zeros(10, dtype=torch.int64, device=dev)
        return dict(p=p, work=work, rec=rec, rec_cap=rec_cap, totals=totals, hits=d_hits, summary=summ, ids=d_ids)

    def grep(self, dict_path, list_path, hits=False, chunk=16384, grid=None, block=128, keep_open=False,
             pair_cap=1 << 23, hit_cap=None, stream=None, sync=True, state=None, corpus_cap=1 << 34,
             rec_cap=1 << 22, file_ids=None, whole_max=0, scan=0):
        """grep -w. Returns a dict with records (n,3) sorted by (file, word),
        totals, digest (sum, xor, nhits), hits (n,3) sorted by (file, offset, word) if requested.
        With sync=False, only enqueues and returns the state (read it after synchronising).

        Capacities come from file metadata (stat), never from file contents: the
        contents are read on the GPU through gopen/gread."""
        from . import GREP_SUMMARY, gfs_grep, gfs_grep_graph_launch
        if state is None:
            state = self.grep_state(dict_path, list_path, hits, chunk, grid, block, keep_open, pair_cap, hit_cap,
                                    corpus_cap, rec_cap, file_ids, whole_max, scan)
        p = state["p"]
        s, sp = self._stream(stream)
        if state.get("graph") is not None:  # the run captured by grep_graph (same arguments)
            gfs_grep_graph_launch(state["graph"], sp)
        else:
            gfs_grep(self.h, sp, dict_path, list_path, p, state["work"].data_ptr(), state["rec"].data_ptr(),
                     state["rec_cap"], state["totals"].data_ptr(),
                     state["hits"].data_ptr() if state["hits"] is not None else None, state["summary"].data_ptr())
        if not sync:
            return state
        s.synchronize()
        summ = dict(zip(GREP_SUMMARY, (int(x) for x in state["summary"].cpu().numpy())))
        if summ["err"] == -28 and pair_cap < (1 << 30):  # -ENOSPC: a table was too small
            return self.grep(dict_path, list_path, hits, chunk, grid, block, keep_open, pair_cap * 4, hit_cap,
                             stream, sync, None, corpus_cap * 4, max(rec_cap, summ["nrecords"]) * 2, file_ids,
                             whole_max, scan)
        out = {"summary": summ}
        nrec = min(summ["nrecords"], state["rec_cap"])
        r = state["rec"][:3 * nrec].view(nrec, 3).cpu().numpy().astype(np.uint64)
        order = np.lexsort((r[:, 1], r[:, 0])) if nrec else np.zeros(0, np.int64)
        out["records"] = r[order]
        out["totals"] = state["totals"][:summ["nwords"]].cpu().numpy().astype(np.uint64)
        out["digest"] = (summ["digest_sum"] & ((1 << 64) - 1), summ["digest_xor"] & ((1 << 64) - 1), summ["nhits"])
        if hits:
            nl = min(summ["nhits_listed"], p.hit_cap)
            hv = state["hits"][:2 * nl].view(nl, 2).cpu().numpy().view(np.uint64)
            hh = np.stack([hv[:, 0] >> np.uint64(32), hv[:, 1], hv[:, 0] & np.uint64(0xFFFFFFFF)], axis=1) \
                if nl else np.zeros((0, 3), np.uint64)
            order = np.lexsort((hh[:, 2], hh[:, 1], hh[:, 0])) if nl else np.zeros(0, np.int64)
            out["hits"] = hh[order]
        out["state"] = state
        return out

    def grep_graph(self, state, dict_path, list_path):
        """Capture one grep run with these arguments as a CUDA graph (gfs_grep_graph_create);
        grep(state=state, ...) then replays it (one graph launch instead of ~16 kernel
        launches). Returns the state; close_grep_graph(state) frees the graph."""
        from . import gfs_grep_graph_create
        p = state["p"]
        state["graph"] = gfs_grep_graph_create(
            self.h, None, dict_path, list_path, p, state["work"].data_ptr(), state["rec"].data_ptr(),
            state["rec_cap"], state["totals"].data_ptr(),
            state["hits"].data_ptr() if state["hits"] is not None else None, state["summary"].data_ptr())
        return state

    @staticmethod
    def close_grep_graph(state):
        from . import gfs_grep_graph_destroy
        if state.get("graph") is not None:
            gfs_grep_graph_destroy(state.pop("graph"))

    # mat-vec -------------------------------------------------------------------
    def matvec(self, a_path, x_path, y_path, rows, cols, grid=None, block=256, stream=None, sync=True, state=None,
               row0=0, nrows=None):
        """y = A x through gmmap/gwrite/gfsync for rows [row0, row0 + nrows) of A
        (default: all). Returns (y device tensor, err)."""
        torch = _torch()
        from . import gfs_matvec_rows
        dev = f"cuda:{self.device}"
        nrows = rows - row0 if nrows is None else nrows
        if grid is None:
            grid = max(1, min(nrows, 4 * 148))
            while (nrows + grid - 1) // grid * 4 > 160 * 1024:
                grid *= 2
        if state is None:
            state = dict(x=torch.empty(cols, dtype=torch.float32, device=dev),
                         y=torch.empty(nrows, dtype=torch.float32, device=dev),
                         err=torch.zeros(2, dtype=torch.int64, device=dev))
        s, sp = self._stream(stream)
        gfs_matvec_rows(self.h, sp, a_path, x_path, y_path, rows, cols, row0, nrows, state["x"].data_ptr(),
                        state["y"].data_ptr(), state["err"].data_ptr(), grid, block)
        if not sync:
            return state
        s.synchronize()
        return state["y"], int(state["err"][0].item())

    def pin(self, path, flags=0) -> int:
        """Open `path` and keep it open across launches (later gopen calls need no RPC)."""
        return self.fileop(path, "pin", flags=flags)

    def unpin(self, fd) -> int:
        return self.fileop("", "unpin", arg=fd)

    def gfsync(self, path, flags=1, grid=1):
        """gfsync(path) from one block, or from `grid` blocks at once (+ a strict pass)."""
        if grid > 1:
            return self.fileop(path, "fsync_grid", flags=flags, arg=grid)
        return self.fileop(path, "fsync", flags=flags)

    def gftruncate(self, path, size):
        return self.fileop(path, "ftruncate", flags=1, arg=size)

    def gfstat(self, path, flags=0):
        return self.fileop(path, "fstat", flags=flags)
