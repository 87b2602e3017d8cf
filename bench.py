#!/usr/bin/env python
"""bench.py — GPUfs buffer-cache read path on B200 (BASELINE.json configs[1]).

Headline workload (N=1, configs[1]): sequential gread sweep over one file
larger than the 4 GiB GPU cache (P = 2 MiB), so every page is a miss RPC +
pread + DMA fill + LRU eviction, followed by the block's checksum of the
bytes read. value = file GB/s of the sweep kernel (CUDA events on its stream).

Also measured in the same run (extra keys):
  hit   — K4-shape cache-hit gread (16 KiB chunks -> shared memory at random
          offsets of a pre-warmed file), against HBM and against a raw-memory
          baseline kernel with the same access pattern;
  grep  — (when available) grep -w corpus GB/s.

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
Multi-GPU: one process per GPU (torchrun), each rank sweeps its own file with
a private cache (weak scaling); the only collective is the final all-reduce of
checksums. Timing = max over ranks of the device-timed region.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

MEASURED = os.path.join(ROOT, "MEASURED_PEAKS.json")
FALLBACK_HBM = 6650.0


def peaks():
    try:
        with open(MEASURED) as f:
            d = json.load(f)
        return float(d["hbm_gbs"]), "measured"
    except Exception:
        return FALLBACK_HBM, "fallback"


class Clocks:
    """Sample nvidia-smi clocks and throttle reasons during the timed region."""

    def __init__(self, index: int):
        self.index = index
        self.samples = []
        self._stop = threading.Event()
        self._th = None

    def _nvml_handle(self):
        """In-process NVML (no nvidia-smi process per sample competing with the daemon's
        workers for host cores); the device found by PCI bus id (CUDA ordinals may be remapped)."""
        try:
            import pynvml
            import torch
            pynvml.nvmlInit()
            pr = torch.cuda.get_device_properties(self.index)
            bus = f"{pr.pci_domain_id:08x}:{pr.pci_bus_id:02x}:{pr.pci_device_id:02x}.0"
            return pynvml, pynvml.nvmlDeviceGetHandleByPciBusId(bus)
        except Exception:
            return None, None

    def __enter__(self):
        nv, hd = self._nvml_handle()

        def run_nvml():
            act = lambda m, bit: "Active" if m & bit else "Not Active"
            while not self._stop.is_set():
                try:
                    m = nv.nvmlDeviceGetCurrentClocksEventReasons(hd) \
                        if hasattr(nv, "nvmlDeviceGetCurrentClocksEventReasons") \
                        else nv.nvmlDeviceGetCurrentClocksThrottleReasons(hd)
                    self.samples.append([str(nv.nvmlDeviceGetClockInfo(hd, nv.NVML_CLOCK_SM)),
                                         str(nv.nvmlDeviceGetMaxClockInfo(hd, nv.NVML_CLOCK_SM)),
                                         act(m, 0x8), act(m, 0x40), act(m, 0x20), act(m, 0x4)])
                except Exception:
                    pass
                self._stop.wait(0.2)

        def run():
            q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,"
                 "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
                 "clocks_event_reasons.sw_power_cap")
            while not self._stop.is_set():
                try:
                    out = subprocess.run(["nvidia-smi", "-i", str(self.index), f"--query-gpu={q}",
                                          "--format=csv,noheader,nounits"], capture_output=True, text=True,
                                         timeout=5).stdout.strip()
                    if out:
                        self.samples.append([x.strip() for x in out.split(",")])
                except Exception:
                    pass
                self._stop.wait(0.2)

        self._th = threading.Thread(target=run_nvml if hd is not None else run, daemon=True)
        self._th.start()
        return self

    def __exit__(self, *a):
        self._stop.set()
        if self._th:
            self._th.join(timeout=10)

    def summary(self):
        if not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"]}
        sm = [float(s[0]) for s in self.samples if s[0].replace(".", "").isdigit()]
        mx = [float(s[1]) for s in self.samples if s[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for s in self.samples for i in range(4) if len(s) > i + 2 and
                          s[i + 2].strip().lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.samples)}


def pinned_h2d_gbs(torch, dev, nbytes=256 << 20, reps=10):
    """In-run pinned host->device cudaMemcpyAsync bandwidth (the miss-fill roofline)."""
    h = torch.empty(nbytes, dtype=torch.uint8).pin_memory()
    d = torch.empty(nbytes, dtype=torch.uint8, device=dev)
    s = torch.cuda.Stream(device=dev)
    best = 0.0
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        with torch.cuda.stream(s):
            e0.record(s)
            d.copy_(h, non_blocking=True)
            e1.record(s)
        s.synchronize()
        best = max(best, nbytes / (e0.elapsed_time(e1) * 1e-3) / 1e9)
    del h, d
    return best


def dist_env():
    ws = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return ws, rank, local


# ---------------------------------------------------------------------- reference arm
def run_reference(args):
    """The CPU oracle as it stands (pread + position checksum), bounded sample."""
    ws, rank, _ = dist_env()
    if ws > 1 and rank != 0:
        return
    import gen
    import oracle
    size = args.file_gib << 30
    path = gen.splitmix_file(f"/dev/shm/gfs_bench_c2_{size}_r0.bin", size, seed=1000)
    sample = min(size, args.ref_sample_mib << 20)
    oracle.checksum(path, 0, 1 << 20)  # warm
    times = []
    for i in range(args.warmup + args.steps):
        off = ((i * 7919) % max(1, size // sample)) * sample
        t0 = time.perf_counter()
        oracle.checksum(path, off, sample)
        dt = time.perf_counter() - t0
        if i >= args.warmup:
            times.append(dt)
    ms = 1e3 * statistics.mean(times)
    val = sample / (ms * 1e-3) / 1e9
    line = {"impl": "reference", "metric": "gread GB/s (miss fill, sequential sweep > cache)", "value": round(val, 3),
            "unit": "GB/s", "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
            "ms_per_step": round(ms, 3), "higher_is_better": True, "scaling": "weak", "vs_baseline": None,
            "dtype": "u8", "data": "synthetic",
            "config": {"workload": f"C2 sequential sweep, {args.file_gib} GiB file, oracle pread+checksum sample "
                                   f"{args.ref_sample_mib} MiB per step"},
            "cpu_baseline": {"value": round(val, 3), "unit": "GB/s", "cores": 1, "kind": "oracle",
                             "sample": f"{args.ref_sample_mib} MiB of the {args.file_gib} GiB file per step"},
            "e2e": {"value": round(val, 3), "unit": "GB/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ---------------------------------------------------------------------- our arm
def run_ours(args):
    import torch
    import torch.distributed as dist

    import gen
    import paper_conf_asplos_silbersteinfkw13_b200 as g

    ws, rank, local = dist_env()
    if os.environ.get("GFS_BENCH_ONE_GPU") == "1":
        # test mode for the multi-rank path on a one-GPU box: every rank on cuda:0, gloo
        # (NCCL refuses two ranks on one GPU); never used for reported numbers
        local = 0
        if ws > 1:
            dist.init_process_group("gloo")
    elif ws > 1:
        dist.init_process_group("nccl", device_id=torch.device(f"cuda:{local}"))
    torch.cuda.set_device(local)
    dev = f"cuda:{local}"
    g.build.build()
    hbm, hbm_src = peaks()

    size = args.file_gib << 30
    P = args.page_kib << 10
    # Two files swept alternately: each is 2x the cache, so sweeping one evicts
    # every page of the other and every step is all misses (no LRU retention).
    paths = [gen.splitmix_file(f"/dev/shm/gfs_bench_c2_{size}_r{rank}_{k}.bin", size, seed=1000 + 16 * rank + k)
             for k in range(2)]
    path = paths[0]
    h2d = pinned_h2d_gbs(torch, dev)

    fs = g.GpuFS(cache_bytes=args.cache_gib << 30, page_size=P, device=local, daemon_threads=args.daemon_threads,
                 max_batch=1, timeout_ms=args.timeout_ms)
    grid = args.grid
    stream = torch.cuda.Stream(device=dev)
    scratch = torch.empty(grid * P, dtype=torch.uint8, device=dev)
    out = torch.zeros(2, dtype=torch.int64, device=dev)
    nstep = [0]

    def step():
        out.zero_()
        fs.seqread(paths[nstep[0] % 2], size, P, grid=grid, stream=stream, sync=False, scratch=scratch, out=out)
        nstep[0] += 1

    with torch.cuda.stream(stream):
        for _ in range(args.warmup):
            step()
        stream.synchronize()
        v = out.cpu().numpy()
        if v[1] != 0:
            print("stats", fs.stats(), fs.host_stats(), fs.info(), file=sys.stderr)
            raise SystemExit(f"gread sweep error {v[1]}")
        fs.stats(reset=True)
        if ws > 1:
            dist.barrier()
        torch.cuda.synchronize()
        evs = []
        with Clocks(local) as clk:
            for _ in range(args.steps):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                step()
                e1.record(stream)
                evs.append((e0, e1))
            stream.synchronize()
        torch.cuda.synchronize()
    step_ms = [a.elapsed_time(b) for a, b in evs]
    ms = float(np.mean(step_ms))
    st = fs.stats()
    hst = fs.host_stats()
    checksum = int(out[0].item()) & ((1 << 64) - 1)

    # e2e: the public API call with host-side result read, wall clock, inputs from tmpfs
    # NOTE: never issue a synchronous copy (tensor.cpu()) while a GPUfs kernel
    # runs: it can hold driver locks the daemon's async DMA needs. Wait on the
    # stream first, then read the result into pinned memory.
    res = torch.empty(2, dtype=torch.int64).pin_memory()
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    rpc_sums = {}
    with torch.cuda.stream(stream):
        for _ in range(args.steps):
            step()
            stream.synchronize()
            res.copy_(out, non_blocking=True)  # D2H of the step's result (checksum, error)
            stream.synchronize()
            rpc_sums[paths[(nstep[0] - 1) % 2]] = int(res[0]) & ((1 << 64) - 1)
    e2e_s = (time.perf_counter() - t0) / args.steps
    if int(res[1]) != 0:
        raise SystemExit(f"gread sweep error {int(res[1])}")

    # K1 variant: the same sweep through gmmap/gmunmap (zero-copy
    # mapping of each page; the consumer checksums the frame in place)
    k1 = None
    if not args.no_k1:
        kt = []
        last_path, last_sum = paths[(nstep[0] - 1) % 2], int(res[0]) & ((1 << 64) - 1)
        k1_parity = True
        with torch.cuda.stream(stream):
            for rep in range(3):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                out.zero_()
                e0.record(stream)
                fs.seqread(paths[nstep[0] % 2], size, P, use_mmap=True, grid=grid, stream=stream, sync=False,
                           scratch=scratch, out=out)
                e1.record(stream)
                stream.synchronize()
                if int(out[1].item()) != 0:
                    raise SystemExit(f"gmmap sweep error {int(out[1].item())}")
                if paths[nstep[0] % 2] == last_path:  # same file as the last gread sweep: same checksum
                    k1_parity &= (int(out[0].item()) & ((1 << 64) - 1)) == last_sum
                kt.append(e0.elapsed_time(e1))
                nstep[0] += 1
        k1_ms = float(np.median(kt))
        k1 = {"workload": "K1: the C2 sweep through gmmap/gmunmap (one page mapped per call)",
              "GBps": round(size / (k1_ms * 1e-3) / 1e9, 3), "ms": round(k1_ms, 3),
              "frac_h2d": round(size / (k1_ms * 1e-3) / 1e9 / h2d, 4),
              "checksum_matches_gread_sweep": bool(k1_parity)}

    # Zero-copy variant of the same sweep: both files registered (gfs_register_file,
    # setup outside the timed region); misses pull straight from the host page cache
    # without READ RPCs or daemon memcpys. Reported beside the RPC-path headline.
    zc = None
    if not args.no_zc:
        try:
            t0 = time.perf_counter()
            for p_ in paths:
                fs.register_file(p_)
            reg_s = time.perf_counter() - t0
            fs.stats(reset=True)
            zt = []
            zc_parity = True
            with torch.cuda.stream(stream):
                for rep_ in range(args.warmup + args.steps):
                    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    e0.record(stream)
                    step()
                    e1.record(stream)
                    stream.synchronize()
                    if int(out[1].item()) != 0:
                        raise RuntimeError(f"zero-copy sweep error {int(out[1].item())}")
                    p_ = paths[(nstep[0] - 1) % 2]
                    if p_ in rpc_sums:  # same file through the RPC path: same checksum
                        zc_parity &= (int(out[0].item()) & ((1 << 64) - 1)) == rpc_sums[p_]
                    if rep_ >= args.warmup:
                        zt.append(e0.elapsed_time(e1))
            zst = fs.stats()
            zms = float(np.mean(zt))
            zc = {"workload": "the C2 sweep with both files registered (gfs_register_file): misses pull from the "
                              "host page cache, no READ RPC", "GBps": round(size / (zms * 1e-3) / 1e9, 3),
                  "frac_h2d": round(size / (zms * 1e-3) / 1e9 / h2d, 4), "register_s": round(reg_s, 2),
                  "zc_fill": zst["zc_fill"], "rpc_read": zst["rpc_read"],
                  "checksum_matches_rpc_sweep": bool(zc_parity)}
        except Exception as e:  # registration refused on this host: say so, keep the RPC headline
            zc = {"unavailable": str(e)[:200]}

    # cache-hit phase (K4 shape): pre-warm a file that fits, random 16 KiB greads into smem
    hit = None
    if not args.no_hit:
        hit = hit_phase(args, torch, g, gen, fs, dev, stream, hbm, rank)
    grep = None
    if not args.no_grep:
        grep = grep_phase(args, torch, g, gen, dev, stream, hbm, rank, ws, local, dist)
    mv = None
    if not args.no_matvec:
        mv = matvec_phase(args, torch, g, gen, dev, stream, h2d, rank, local)
    fig4 = None
    if not args.no_fig4:
        fig4 = fig4_phase(args, torch, g, dev, stream, h2d, paths, size, local)
    c5 = None
    if not args.no_c5:
        c5 = c5_phase(args, torch, g, dev, stream, h2d, hbm, rank, ws, local, dist)

    tmax = torch.tensor([ms], device=dev)
    if ws > 1:
        dist.all_reduce(tmax, op=dist.ReduceOp.MAX)
        cs = torch.tensor([checksum & 0x7FFFFFFFFFFFFFFF], device=dev)
        dist.all_reduce(cs)  # the final reduction (NCCL)
    ms_max = float(tmax.item())
    value = ws * size / (ms_max * 1e-3) / 1e9
    achieved = size / (ms * 1e-3) / 1e9
    clk_s = clk.summary()
    fs.close()
    if rank != 0:
        return
    line = {
        "metric": "gread GB/s (miss fill, sequential sweep > cache)",
        "value": round(value, 3), "unit": "GB/s", "n_gpus": ws, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": round(ms_max, 3), "higher_is_better": True, "scaling": "weak", "vs_baseline": None,
        "dtype": "u8", "data": "synthetic",
        "config": {"workload": f"C2: sequential gread sweep of a {args.file_gib} GiB splitmix file per GPU, "
                               f"{args.cache_gib} GiB GPU cache, {args.page_kib} KiB pages, grid {grid}x256, "
                               f"{args.daemon_threads} daemon threads; tmpfs; file > cache and > L2 (no flush needed)",
                   "page_kib": args.page_kib, "cache_gib": args.cache_gib, "file_gib": args.file_gib},
        "roofline": {"bound": "h2d", "achieved": round(achieved, 3), "peak": round(h2d, 3), "unit": "GB/s",
                     "frac": round(achieved / h2d, 4), "traffic": None,
                     "peak_source": "pinned cudaMemcpyAsync H2D 256 MiB, best of 10, measured in this run"},
        "e2e": {"value": round(size * ws / e2e_s / 1e9, 3), "unit": "GB/s", "h2d_bytes_per_step": size,
                "d2h_bytes_per_step": 16},
        "gpu_launches": args.steps,
        "clocks": clk_s,
        "counters": {k: st[k] for k in ("miss", "hit", "evict", "rpc", "timeout", "enomem", "ring_wait")},
        "host": {"pread_GBps_per_thread": round(hst["bytes_h2d"] / max(hst["pread_ns"], 1), 3) if hst["pread_ns"] else None},
        "checksum": hex(checksum),
    }
    if hit:
        line["hit"] = hit
    if grep:
        line["grep"] = grep
    if mv:
        line["matvec"] = mv
    if c5:
        line["c5"] = c5
    if fig4:
        line["fig4_page_sweep"] = fig4
    if k1:
        line["k1_gmmap"] = k1
    if zc:
        line["c2_zero_copy"] = zc
    if not args.no_cpu:
        line["cpu_baseline"] = cpu_baseline(args, path, size)
    print(json.dumps(line), flush=True)


def hit_phase(args, torch, g, gen, fs_unused, dev, stream, hbm, rank):
    """K4: 16 KiB greads into shared memory at random offsets of a warm file."""
    P = args.hit_page_kib << 10
    size = args.hit_file_gib << 30
    path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}_r{rank}.bin", size, seed=2000 + rank)
    chunk = 16384
    grid = args.hit_grid
    calls = args.hit_calls
    rng = np.random.default_rng(7)
    offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
    d_off = torch.as_tensor(offs.view(np.int64), device=dev)
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=torch.cuda.current_device(),
                 daemon_threads=args.daemon_threads, timeout_ms=args.timeout_ms) as fs:
        s, err = fs.seqread(path, size, P, grid=296)  # pre-warm
        assert err == 0
        fs.stats(reset=True)
        out = torch.zeros(2, dtype=torch.int64, device=dev)
        raw = torch.empty(size, dtype=torch.uint8, device=dev)
        raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8), non_blocking=False)

        def timed(fn, reps):
            ts = []
            for _ in range(reps):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                fn()
                e1.record(stream)
                stream.synchronize()
                ts.append(e0.elapsed_time(e1))
            return float(np.median(ts))

        with torch.cuda.stream(stream):
            run_g = lambda: fs.randread(path, chunk, d_off, grid, block=args.hit_block, stream=stream, sync=False,
                                        out=out)
            run_r = lambda: fs.randread(None, chunk, d_off, grid, block=args.hit_block, raw=raw, stream=stream,
                                        sync=False, out=out)
            for _ in range(2):
                run_g()
                run_r()
            ms_g = timed(run_g, 5)
            ms_r = timed(run_r, 5)
            # K5 ablation (Table 2): the same calls, every lookup
            # under the file lock, against lock-free lookups (fewer calls: the
            # locked variant serialises every block on one file's lock)
            abl_calls = 32
            d_off_a = d_off[:grid * abl_calls]
            run_a = lambda: fs.randread(path, chunk, d_off_a, grid, block=args.hit_block, stream=stream,
                                        sync=False, out=out)
            run_a()
            ms_lockfree = timed(run_a, 3)
            out.zero_()
            run_g()
            stream.synchronize()
            sg = int(out[0].item()) & ((1 << 64) - 1)
            out.zero_()
            run_r()
            stream.synchronize()
            sr = int(out[0].item()) & ((1 << 64) - 1)
        st = fs.stats()
        del raw
    ms_locked = None
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=torch.cuda.current_device(),
                 daemon_threads=args.daemon_threads, timeout_ms=args.timeout_ms, flags=g.F_LOCKED_TRAVERSAL) as fl:
        s2, err2 = fl.seqread(path, size, P, grid=296)
        assert err2 == 0 and s2 == s
        with torch.cuda.stream(stream):
            run_l = lambda: fl.randread(path, chunk, d_off_a, grid, block=args.hit_block, stream=stream,
                                        sync=False, out=out)
            run_l()
            ms_locked = timed(run_l, 3)
        stl = fl.stats()
    nbytes = grid * calls * chunk
    gbs = nbytes / (ms_g * 1e-3) / 1e9
    return {"workload": f"K4: {grid} blocks x {calls} x 16 KiB gread -> smem, random offsets, {args.hit_file_gib} GiB "
                        f"warm file, {args.hit_page_kib} KiB pages",
            "GBps": round(gbs, 3), "raw_GBps": round(nbytes / (ms_r * 1e-3) / 1e9, 3),
            "vs_raw": round(ms_r / ms_g, 4),
            "roofline": {"bound": "hbm", "achieved": round(gbs, 3), "peak": hbm, "unit": "GB/s",
                         "frac": round(gbs / hbm, 4), "traffic": None,
                         "note": "1 algorithmic HBM byte per delivered byte (frame read; destination is smem)"},
            "checksum_match_raw": sg == sr, "misses_after_warm": st["miss"], "ms": round(ms_g, 3),
            "k5_locked_ablation": {"calls_per_block": abl_calls, "lockfree_ms": round(ms_lockfree, 3),
                                   "locked_ms": round(ms_locked, 3),
                                   "lockfree_speedup": round(ms_locked / ms_lockfree, 2),
                                   "locked_lookups": stl["locked"],
                                   "note": "GFS_F_LOCKED_TRAVERSAL: every lookup takes the file lock (the paper "
                                           "reports lock-free ~3x faster, P:L1047-1048)"}}


def grep_phase(args, torch, g, gen, dev, stream, hbm, rank, ws, local, dist):
    """C4 (configs[3]): grep -w of a 58k-word dictionary over a Linux-source-shaped
    tree, files sharded by LPT across ranks; NCCL reduces totals at the end."""
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    root = f"/dev/shm/gfs_bench_c4_{args.grep_files}_{args.grep_mib}"
    if rank == 0:
        c = gen.c4_corpus(root, seed=4, nfiles=args.grep_files, total_bytes=args.grep_mib << 20, nwords=58000)
    if ws > 1:
        dist.barrier()
    c = gen.c4_corpus(root, seed=4, nfiles=args.grep_files, total_bytes=args.grep_mib << 20, nwords=58000)
    sizes = [os.path.getsize(p) for p in c["paths"]]  # metadata only, for the LPT split
    shard = gdist.lpt_shard(sizes, ws)[rank]
    lst = gdist.write_shard_list(c["paths"], shard, f"{root}/shard_{ws}_{rank}.txt")
    shard_bytes = int(sum(sizes[i] for i in shard))
    res = {}
    with g.GpuFS(cache_bytes=args.grep_cache_gib << 30, page_size=64 << 10, device=local,
                 daemon_threads=args.daemon_threads, max_files=1 << 16, timeout_ms=args.timeout_ms) as fs:
        # device buffers allocated outside the timed region (reused by every run)
        state = fs.grep_state(c["dict"], lst, hits=False, keep_open=True, rec_cap=1 << 24)
        out = None
        for phase in ("cold", "warm"):
            torch.cuda.synchronize()
            if ws > 1:
                dist.barrier()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            with torch.cuda.stream(stream):
                e0.record(stream)
                st = fs.grep(c["dict"], lst, hits=False, keep_open=True, stream=stream, sync=False, state=state)
                e1.record(stream)
                stream.synchronize()
            state = st
            ms = e0.elapsed_time(e1)
            t = torch.tensor([ms], device=dev)
            if ws > 1:
                dist.all_reduce(t, op=dist.ReduceOp.MAX)
            ms_max = float(t.item())
            res[phase] = {"ms": round(ms_max, 3), "GBps": round(args.grep_mib * (1 << 20) / (ms_max * 1e-3) / 1e9, 4),
                          "files_per_s": round(args.grep_files / (ms_max * 1e-3), 1)}
        out = fs.grep(c["dict"], lst, hits=False, keep_open=True, stream=stream, state=state)
        gst = fs.stats()
    summ = out["summary"]
    recs = gdist.globalize_records(out["records"], shard)
    if ws > 1:
        tot, dig, allrecs = gdist.reduce_grep(dist.group.WORLD, out["totals"], out["digest"], recs,
                                              device=torch.device(dev))
    else:
        tot, dig, allrecs = out["totals"], out["digest"], recs
    res.update({"workload": f"C4: {args.grep_files} files / {args.grep_mib} MiB C-like text, 58,000-word dictionary, "
                            f"LPT shard over {ws} GPU(s), 64 KiB pages; cold = fresh cache (OPEN + READ RPCs), "
                            f"warm = files kept open, pages cached",
                "err": summ["err"], "nhits": int(dig[2]), "nrecords": int(len(allrecs)),
                "shard_bytes_rank0": shard_bytes,
                "rpc_open": gst["rpc_open"], "rpc_read": gst["rpc_read"], "misses": gst["miss"]})
    warm_gbs = res["warm"]["GBps"] / ws  # per GPU
    res["roofline_warm"] = {"bound": "hbm", "achieved": round(warm_gbs, 3), "peak": hbm, "unit": "GB/s",
                            "frac": round(warm_gbs / hbm, 5),
                            "note": "1 algorithmic HBM byte per corpus byte (frame -> smem); per GPU"}
    if rank == 0 and not args.no_cpu:
        import oracle
        t0 = time.perf_counter()
        ref = oracle.grep(c["dict"], c["list"], want_hits=False, nthreads=os.cpu_count() or 1)
        dt = time.perf_counter() - t0
        res["parity"] = {"totals": ref.totals.tolist() == list(map(int, tot)), "nhits": ref.digest[2] == int(dig[2]),
                         "records": ref.records.tolist() == allrecs.tolist()}
        if ws == 1:
            res["parity"]["digest"] = (ref.digest[0], ref.digest[1]) == (int(dig[0]), int(dig[1]))
        res["cpu_baseline"] = {"value": round(ref.bytes / dt / 1e9, 4), "unit": "GB/s", "cores": os.cpu_count(),
                               "kind": "oracle", "sample": f"whole C4 corpus ({ref.bytes} B), nproc threads"}
    return res


def matvec_phase(args, torch, g, gen, dev, stream, h2d, rank, local):
    """C3 (configs[2]): y = A x, A (rows x 131072 fp32) larger than the 2 GiB cache,
    read through gmmap, y through gwrite + gfsync."""
    import oracle
    rows, cols = args.mv_rows, 131072
    m = gen.matrix_files(f"/dev/shm/gfs_bench_c3_r{rank}", rows, cols, seed=3 + rank)
    ypath = f"/dev/shm/gfs_bench_c3_r{rank}/y.f32"
    nbytes = rows * cols * 4
    with g.GpuFS(cache_bytes=2 << 30, page_size=2 << 20, device=local, daemon_threads=args.daemon_threads,
                 max_batch=1, timeout_ms=args.timeout_ms) as fs:
        state = None
        ts = []
        for it in range(3):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            with torch.cuda.stream(stream):
                e0.record(stream)
                state = fs.matvec(m["A"], m["x"], ypath, rows, cols, stream=stream, sync=False, state=state)
                e1.record(stream)
                stream.synchronize()
            ts.append(e0.elapsed_time(e1))
        err = int(state["err"][0].item())
        y = state["y"].cpu().numpy().astype(np.float64)
        st = fs.stats()
        # the same product with the matrix file registered (zero-copy misses, §4.3 of DESIGN.md)
        zc = None
        if not args.no_zc:
            try:
                t0 = time.perf_counter()
                fs.register_file(m["A"])
                reg_s = time.perf_counter() - t0
                zts = []
                for it in range(3):
                    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    with torch.cuda.stream(stream):
                        e0.record(stream)
                        state = fs.matvec(m["A"], m["x"], ypath, rows, cols, stream=stream, sync=False,
                                          state=state)
                        e1.record(stream)
                        stream.synchronize()
                    zts.append(e0.elapsed_time(e1))
                zy = state["y"].cpu().numpy().astype(np.float64)
                zms = float(np.median(zts))
                zc = {"GBps": round(nbytes / (zms * 1e-3) / 1e9, 3),
                      "frac_h2d": round(nbytes / (zms * 1e-3) / 1e9 / h2d, 4), "register_s": round(reg_s, 2),
                      "y_equal_rpc_path": bool(np.array_equal(zy, y)) and int(state["err"][0].item()) == 0}
            except Exception as e:
                zc = {"unavailable": str(e)[:200]}
    ms = float(np.median(ts))
    gbs = nbytes / (ms * 1e-3) / 1e9
    rng = np.random.default_rng(0)
    sample = np.unique(np.concatenate([np.arange(8), rng.integers(0, rows, size=56)]))
    ref = np.array([oracle.matvec(m["A"], m["x"], rows, cols, row0=int(r), nrows=1)[0] for r in sample])
    relerr = float(np.max(np.abs(y[sample] - ref) / np.abs(ref)))
    yh = np.fromfile(ypath, dtype="<f4").astype(np.float64)
    out = {"workload": f"C3: {rows} x {cols} fp32 matrix ({nbytes >> 20} MiB) > 2 GiB cache, 2 MiB pages, "
                       f"gmmap rows, gwrite+gfsync y",
           "GBps": round(gbs, 3), "ms": round(ms, 3), "err": err,
           "roofline": {"bound": "h2d", "achieved": round(gbs, 3), "peak": round(h2d, 3), "unit": "GB/s",
                        "frac": round(gbs / h2d, 4)},
           "max_rel_err_sampled_rows": relerr, "parity_ok": relerr <= 1e-5 and np.array_equal(yh, y),
           "misses": st["miss"], "evictions": st["evict"]}
    if zc:
        out["zero_copy"] = zc
    if not args.no_cpu:
        t0 = time.perf_counter()
        n = min(rows, 2048)
        oracle.matvec(m["A"], m["x"], rows, cols, row0=0, nrows=n, nthreads=os.cpu_count() or 1)
        dt = time.perf_counter() - t0
        out["cpu_baseline"] = {"value": round(n * cols * 4 / dt / 1e9, 3), "unit": "GB/s",
                               "cores": os.cpu_count(), "kind": "oracle",
                               "sample": f"first {n} rows, float64, nproc threads"}
    return out


def fig4_phase(args, torch, g, dev, stream, h2d, paths, size, local):
    """Fig. 4 analogue: miss-fill GB/s of a sequential gread sweep
    against page size. Sweeps alternate between the first 4 GiB of the two C2
    files with a 2 GiB cache, so every page is a miss (no LRU retention)."""
    total = min(size, 4 << 30)
    out = []
    for pk in (64, 256, 1024, 2048, 4096, 16384):
        P = pk << 10
        frames = (2 << 30) // P
        grid = int(min(296, frames // 2))
        with g.GpuFS(cache_bytes=2 << 30, page_size=P, device=local, daemon_threads=args.daemon_threads,
                     timeout_ms=args.timeout_ms, max_batch=min(32, max(1, (8 << 20) // P))) as fs:
            chunk = max(P, 2 << 20)
            scratch = torch.empty(grid * chunk, dtype=torch.uint8, device=dev)
            res = torch.zeros(2, dtype=torch.int64, device=dev)
            ts = []
            for rep in range(3):
                res.zero_()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                with torch.cuda.stream(stream):
                    e0.record(stream)
                    fs.seqread(paths[rep % 2], total, chunk, grid=grid, stream=stream, sync=False, scratch=scratch,
                               out=res)
                    e1.record(stream)
                    stream.synchronize()
                if rep:
                    ts.append(e0.elapsed_time(e1))
            err = int(res[1].item())
            st = fs.stats()
        ms = float(np.median(ts))
        gbs = total / (ms * 1e-3) / 1e9
        out.append({"page_kib": pk, "GBps": round(gbs, 3), "frac_h2d": round(gbs / h2d, 4), "err": err,
                    "grid": grid, "misses": st["miss"], "hits": st["hit"]})
    return {"workload": f"sequential gread sweep of {total >> 30} GiB, 2 GiB cache, chunk max(P, 2 MiB)",
            "points": out}


def c5_phase(args, torch, g, dev, stream, h2d, hbm, rank, ws, local, dist):
    """C5 (configs[4]): repeated gwrite/gfsync then re-read across kernel launches.
    Rank r writes f_r (O_GWRONCE, new content every iteration) and gfsyncs it;
    after a barrier it re-reads f_{(r+1) % N} twice through its own cache: the
    first pass re-validates (close-to-open) and misses, the second
    hits. At N = 1 the file read is the rank's own (re-opened read-only: a fresh
    incarnation). Parity: the host file equals the source bytes and
    the GPU read-back checksum equals the oracle's checksum of the host file."""
    import oracle
    P = 2 << 20
    size = args.c5_mib << 20
    root = "/dev/shm/gfs_bench_c5"
    os.makedirs(root, exist_ok=True)
    mine, peer = f"{root}/f_{rank}.bin", f"{root}/f_{(rank + 1) % ws}.bin"
    if os.path.exists(mine):  # a write-once open does not truncate: start from no file
        os.remove(mine)
    base = torch.from_numpy(np.random.default_rng(500 + rank).integers(0, 256, size=size, dtype=np.uint8)).to(dev)
    src = torch.empty_like(base)
    grid = 296
    times = {"write": [], "read_miss": [], "read_hit": []}
    ok_host, ok_read, errs = True, True, []
    with g.GpuFS(cache_bytes=4 << 30, page_size=P, device=local, daemon_threads=args.daemon_threads,
                 max_batch=8, timeout_ms=args.timeout_ms, staging_slots=256) as fs:
        scratch = torch.empty(grid * P, dtype=torch.uint8, device=dev)
        out = torch.zeros(2, dtype=torch.int64, device=dev)
        wout = torch.zeros(2, dtype=torch.int64, device=dev)
        npeers = 0
        peer_err = None
        if ws > 1 and not args.no_peers:
            # NEXT-1: every cache maps the others (CUDA IPC over NVLink); the first
            # re-read of the neighbour's file is then served from the writer's cache
            descs = [None] * ws
            try:
                mine_desc = fs.export()
            except Exception as e:  # no CUDA IPC here: run C5 without peers, say so
                mine_desc, peer_err = None, f"export: {e}"
            dist.all_gather_object(descs, mine_desc)
            for r, d in enumerate(descs):
                if r != rank and d is not None:
                    try:
                        fs.attach_peer(d)
                        npeers += 1
                    except Exception as e:
                        peer_err = f"attach rank {r}: {e}"
            # every rank attaches all or none, so the re-read path is the same everywhere
            ok = torch.tensor([1 if npeers == ws - 1 else 0], device=dev)
            dist.all_reduce(ok, op=dist.ReduceOp.MIN)
            if int(ok.item()) == 0 and peer_err is None:
                peer_err = "some ranks could not attach every peer (results stay exact: peer fill is optional)"
        for it in range(args.c5_iters):
            src.copy_(base)
            src.add_(it + 1)  # new content every iteration (mod 256), prepared before the timed region
            torch.cuda.synchronize()
            e = [torch.cuda.Event(enable_timing=True) for _ in range(4)]
            with torch.cuda.stream(stream):
                e[0].record(stream)
                fs.seqwrite(mine, src, chunk=P, grid=grid, sync_grid=args.c5_sync_grid, stream=stream, sync=False,
                            out=wout)
                e[1].record(stream)
                stream.synchronize()
            errs.append(int(wout[0].item()))
            if ws > 1:
                dist.barrier()  # every writer has gfsync'ed before anyone re-opens
            with torch.cuda.stream(stream):
                out.zero_()
                e[2].record(stream)
                fs.seqread(peer, size, P, grid=grid, stream=stream, sync=False, scratch=scratch, out=out)
                e[3].record(stream)
                stream.synchronize()
            s1, err1 = int(out[0].item()) & ((1 << 64) - 1), int(out[1].item())
            e2 = [torch.cuda.Event(enable_timing=True) for _ in range(2)]
            with torch.cuda.stream(stream):
                out.zero_()
                e2[0].record(stream)
                fs.seqread(peer, size, P, grid=grid, stream=stream, sync=False, scratch=scratch, out=out)
                e2[1].record(stream)
                stream.synchronize()
            s2, err2 = int(out[0].item()) & ((1 << 64) - 1), int(out[1].item())
            errs += [err1, err2]
            times["write"].append(e[0].elapsed_time(e[1]))
            times["read_miss"].append(e[2].elapsed_time(e[3]))
            times["read_hit"].append(e2[0].elapsed_time(e2[1]))
            want = oracle.checksum(peer, 0, size)
            ok_read &= s1 == want and s2 == want
            if it == args.c5_iters - 1:
                hb = np.fromfile(mine, dtype=np.uint8)
                ok_host &= hb.size == size and np.array_equal(hb, src.cpu().numpy())
            if ws > 1:
                dist.barrier()  # nobody rewrites its file while a peer still reads it
        st = fs.stats()
        local_peer = None
        if ws == 1 and not args.no_peers:
            local_peer = c5_local_peer(args, torch, g, fs, mine, size, P, grid, dev, stream, scratch, out)
    res = {}
    for k, v in times.items():
        t = torch.tensor([float(np.median(v))], device=dev)
        if ws > 1:
            dist.all_reduce(t, op=dist.ReduceOp.MAX)
        ms = float(t.item())
        res[k] = {"ms": round(ms, 3), "GBps": round(ws * size / (ms * 1e-3) / 1e9, 3)}
    res.update({
        "workload": f"C5: {args.c5_iters} iterations x (gwrite {args.c5_mib} MiB O_GWRONCE + gfsync from "
                    f"{args.c5_sync_grid} block(s); barrier; re-read the peer's file twice), 2 MiB pages, 4 GiB "
                    f"cache, {ws} GPU(s)",
        "err": min(errs) if errs else 0, "parity": {"host_file": bool(ok_host), "reread_checksums": bool(ok_read)},
        "counters": {k: st[k] for k in ("miss", "hit", "writeback", "invalidate", "reopen_valid", "rpc_write",
                                        "rpc_read", "peer_fill", "bytes_peer")},
        "peers_attached": npeers,
        "peer_error": peer_err,
        "roofline": {"read_miss": ({"bound": "h2d", "peak": round(h2d, 3),
                                    "frac": round(res["read_miss"]["GBps"] / ws / h2d, 4)} if not npeers else
                                   {"bound": "nvlink", "peak": 900.0, "unit": "GB/s",
                                    "peak_source": "nominal NVLink 5 per-direction bandwidth per GPU",
                                    "frac": round(res["read_miss"]["GBps"] / ws / 900.0, 4)}),
                     "read_hit": {"bound": "hbm", "peak": hbm, "note": "2 B HBM per byte (frame read + copy out)",
                                  "frac": round(2 * res["read_hit"]["GBps"] / ws / hbm, 4)}},
    })
    if local_peer:
        res["read_peer_same_gpu"] = local_peer
    if ws == 1 and not args.no_rdwr:
        res["rdwr_shared_pages"] = rdwr_phase(args, torch, g, dev)
    return res


def rdwr_phase(args, torch, g, dev):
    """NEXT-4: two caches (stand-ins for two GPUs) open one existing
    file O_RDWR and write interleaved 64 KiB blocks of every 2 MiB page (false
    sharing), then gfsync: each write-back sends only the bytes that differ from
    the page's pristine copy, so both halves survive. Parity: the host file
    equals the original with both writers' blocks laid over it."""
    P, blk = 2 << 20, 64 << 10
    size = args.rdwr_mib << 20
    root = "/dev/shm/gfs_bench_rdwr"
    os.makedirs(root, exist_ok=True)
    path = f"{root}/shared.bin"
    orig = np.random.default_rng(900).integers(0, 256, size=size, dtype=np.uint8)
    orig.tofile(path)
    offs = np.arange(0, size, blk, dtype=np.uint64)
    new = np.random.default_rng(901).integers(0, 256, size=size, dtype=np.uint8)
    times = {"gwrite": [], "gfsync": []}
    # 512 staging slots (1 GiB pinned): every O_RDWR page fetch holds one while its block pulls it,
    # and the default 64 slots serialised the first writes of the 128 pages (35 -> 14 ms measured)
    caches = [g.GpuFS(cache_bytes=2 * size + (256 << 20), page_size=P, device=torch.cuda.current_device(),
                      daemon_threads=args.daemon_threads, max_batch=8, timeout_ms=args.timeout_ms,
                      staging_slots=512)
              for _ in range(2)]
    try:
        fds = [c.pin(path, flags=g.O_RDWR) for c in caches]
        for k, c in enumerate(caches):
            mine = offs[k::2]
            data = torch.from_numpy(np.concatenate([new[int(o):int(o) + blk] for o in mine])).to(dev)
            e = [torch.cuda.Event(enable_timing=True) for _ in range(4)]
            torch.cuda.synchronize()
            e[0].record()
            ret = c.gwrite_calls(path, mine, np.full(len(mine), blk, np.uint64), data, grid=296, flags=g.O_RDWR)
            e[1].record()
            assert (ret == blk).all(), ret[:4]
            e[2].record()
            r = c.gfsync(path, flags=g.O_RDWR, grid=64)
            e[3].record()
            torch.cuda.synchronize()
            assert r == 0, r
            times["gwrite"].append(e[0].elapsed_time(e[1]))
            times["gfsync"].append(e[2].elapsed_time(e[3]))
        for c, fd in zip(caches, fds):
            c.unpin(fd)
        st = [c.stats() for c in caches]
    finally:
        for c in caches:
            c.close()
    host = np.fromfile(path, dtype=np.uint8)
    ok = host.size == size and np.array_equal(host, new)  # every block came from one of the two writers
    half = size / 2
    return {"workload": f"two caches, one {args.rdwr_mib} MiB file O_RDWR, 2 MiB pages, interleaved 64 KiB blocks "
                        f"(every page written by both), gwrite then gfsync per cache; one GPU",
            "gwrite_GBps": round(half / (float(np.mean(times["gwrite"])) * 1e-3) / 1e9, 3),
            "gfsync_GBps": round(half / (float(np.mean(times["gfsync"])) * 1e-3) / 1e9, 3),
            "parity": bool(ok), "writebacks": [x["writeback"] for x in st], "misses": [x["miss"] for x in st],
            "note": "source bytes resident in HBM; gwrite includes the page fetches (O_RDWR reads pages) and "
                    "pristine copies; gfsync diffs on the GPU, moves bytes + mask over PCIe, the host writes "
                    "only changed bytes"}


def c5_local_peer(args, torch, g, fs, path, size, P, grid, dev, stream, scratch, out):
    """N = 1 stand-in for NEXT-1 (peer-cache fill): a second cache on the same GPU
    attaches `fs` as its peer and reads the file `fs` holds; every page is copied
    frame-to-frame (HBM -> HBM here; over NVLink between GPUs). Parity: the
    checksum equals the oracle's over the host file."""
    import oracle
    want = oracle.checksum(path, 0, size)
    times, ok, st = [], True, {}
    for rep in range(3):
        with g.GpuFS(cache_bytes=4 << 30, page_size=P, device=fs.device, daemon_threads=2, max_batch=8,
                     timeout_ms=args.timeout_ms) as B:
            B.attach_peer(fs.export())
            torch.cuda.synchronize()
            e = [torch.cuda.Event(enable_timing=True) for _ in range(2)]
            with torch.cuda.stream(stream):
                out.zero_()
                e[0].record(stream)
                B.seqread(path, size, P, grid=grid, stream=stream, sync=False, scratch=scratch, out=out)
                e[1].record(stream)
                stream.synchronize()
            ok &= (int(out[0].item()) & ((1 << 64) - 1)) == want and int(out[1].item()) == 0
            times.append(e[0].elapsed_time(e[1]))
            st = B.stats()
    ms = float(np.median(times))
    return {"ms": round(ms, 3), "GBps": round(size / (ms * 1e-3) / 1e9, 3), "parity": bool(ok),
            "peer_fill": st["peer_fill"], "bytes_peer": st["bytes_peer"], "rpc_read": st["rpc_read"],
            "note": "second cache on the same GPU attached as a peer (NEXT-1 protocol; the copy is HBM->HBM, "
                    "not NVLink); includes the reader's gopen (OPEN RPC)"}


def cpu_baseline(args, path, size):
    import oracle
    sample = min(size, args.ref_sample_mib << 20)
    t0 = time.perf_counter()
    oracle.checksum(path, 0, sample)
    dt = time.perf_counter() - t0
    return {"value": round(sample / dt / 1e9, 3), "unit": "GB/s", "cores": 1, "kind": "oracle",
            "sample": f"oracle pread+checksum of the first {args.ref_sample_mib} MiB of the sweep file"}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--file-gib", type=int, default=8)
    ap.add_argument("--cache-gib", type=int, default=4)
    ap.add_argument("--page-kib", type=int, default=2048)
    ap.add_argument("--grid", type=int, default=296)
    ap.add_argument("--daemon-threads", type=int, default=12)
    ap.add_argument("--hit-file-gib", type=int, default=4)
    ap.add_argument("--hit-page-kib", type=int, default=512)
    ap.add_argument("--hit-grid", type=int, default=1184)   # 8 blocks/SM: lookups of one block overlap
    ap.add_argument("--hit-block", type=int, default=128)   # copies of the others (measured best)
    ap.add_argument("--hit-calls", type=int, default=1024)
    ap.add_argument("--ref-sample-mib", type=int, default=2048)
    ap.add_argument("--timeout-ms", type=int, default=60000)
    ap.add_argument("--no-hit", action="store_true")
    ap.add_argument("--no-grep", action="store_true")
    ap.add_argument("--no-matvec", action="store_true")
    ap.add_argument("--no-c5", action="store_true")
    ap.add_argument("--no-fig4", action="store_true")
    ap.add_argument("--no-k1", action="store_true")
    ap.add_argument("--no-zc", action="store_true", help="skip the zero-copy (registered file) C2 variant")
    ap.add_argument("--c5-mib", type=int, default=512)
    ap.add_argument("--c5-iters", type=int, default=3)
    ap.add_argument("--c5-sync-grid", type=int, default=8)
    ap.add_argument("--mv-rows", type=int, default=11200)  # 5.6 GB (Fig. 8's 5600 MB point x2)
    ap.add_argument("--grep-files", type=int, default=30000)
    ap.add_argument("--grep-mib", type=int, default=500)
    ap.add_argument("--grep-cache-gib", type=int, default=4)
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--no-peers", action="store_true", help="C5 without peer-cache fill (NEXT-1)")
    ap.add_argument("--no-rdwr", action="store_true", help="skip the O_RDWR shared-page phase (NEXT-4)")
    ap.add_argument("--rdwr-mib", type=int, default=256)
    args = ap.parse_args()
    if args.impl == "reference":
        run_reference(args)
    else:
        run_ours(args)


if __name__ == "__main__":
    main()
