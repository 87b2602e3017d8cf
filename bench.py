#!/usr/bin/env python
"""bench.py — GPUfs buffer-cache read path on B200 (BASELINE.json configs[1]).

Headline workload (N=1, configs[1]): sequential gread sweep over one file
larger than the 4 GiB GPU cache (P = 2 MiB), so every page is a miss RPC +
pread + pull into a frame + LRU eviction, followed by the block's checksum of
the bytes read. value = file GB/s of the sweep kernel (CUDA events on its
stream), mean of the K timed steps (stddev reported).

Every phase checks its result against the CPU oracle (oracle/) at the size it
was timed at and reports `parity`:
  C2   sweep checksum == oracle checksum of the whole file (threaded oracle)
  K1   the same sweep through gmmap; zero-copy variant (registered files)
  K4   cache-hit gread -> shared memory (16 KiB, random offsets): checksum ==
       oracle sum over the same calls; raw-memory baseline kernel beside it
  HG   cache-hit gread -> global (256 KiB - 2 MiB chunks, warm 16 GiB file):
       destination checksum == oracle checksum of the file
  C3   out-of-core mat-vec, a FRESH cache per pass (every page a miss): all
       rows vs the float64 oracle (<= 1e-5 relative), y file == y
  C1   grep -w, 64 words x 8 MiB: records, totals, digest and the full hit list
  C4   grep -w, 58k words x 30k files: records, totals, digest (global file ids)
  C5   gwrite/gfsync + re-read: host file bytes, re-read checksums
Multi-GPU (torchrun, one process per GPU): every rank sweeps the same
read-only inputs with its private cache (weak scaling); C3 is row-sharded and
its y shards are all-gathered (NCCL); C4 is file-sharded (LPT) and reduced
(NCCL all-reduce of totals, records gathered to rank 0); a C2 byte-range split
of one file is timed beside the headline. Timing = max over ranks.

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
"""
from __future__ import annotations

import argparse
import json
import os
import shutil
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

# Load every kernel when the CUDA context is created (not at its first launch):
# a "cold" grep or fill then measures the cache, not lazy module loading.
os.environ.setdefault("CUDA_MODULE_LOADING", "EAGER")

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

MEASURED = os.path.join(ROOT, "MEASURED_PEAKS.json")
FALLBACK_HBM = 6650.0
SHM = "/dev/shm"
M64 = (1 << 64) - 1


def peaks():
    try:
        with open(MEASURED) as f:
            d = json.load(f)
        return float(d["hbm_gbs"]), "measured"
    except Exception:
        return FALLBACK_HBM, "fallback"


def mstd(xs):
    """mean and sample stddev of a list (stddev 0 for one sample)."""
    xs = [float(x) for x in xs]
    return (statistics.mean(xs), statistics.stdev(xs) if len(xs) > 1 else 0.0)


def gbs(nbytes, ms):
    return nbytes / (ms * 1e-3) / 1e9


class Clocks:
    """Sample SM clocks and throttle reasons during the timed region (NVML in-process)."""

    def __init__(self, index: int):
        self.index = index
        self.samples = []
        self._stop = threading.Event()
        self._th = None

    def _nvml_handle(self):
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
    """The host->device link (the miss-fill roofline): best of `reps` of the copy engine
    (cudaMemcpyAsync) and of SMs pulling mapped pinned memory the way gread pulls staging
    slots (gfs_probe_h2d); returns (peak = the faster, copy-engine GB/s, SM-pull GB/s)."""
    from paper_conf_asplos_silbersteinfkw13_b200 import gfs_probe_h2d
    s = torch.cuda.Stream(device=dev)
    with torch.cuda.device(dev):
        ce, sm = gfs_probe_h2d(s.cuda_stream, nbytes, reps)
    return max(ce, sm), ce, sm


def dist_env():
    ws = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return ws, rank, local


class Ctx:
    """What every phase needs: torch, the package, the process group, the stream."""

    def __init__(self, args):
        import torch
        import torch.distributed as dist

        import gen
        import paper_conf_asplos_silbersteinfkw13_b200 as g
        self.torch, self.dist, self.gen, self.g, self.args = torch, dist, gen, g, args
        self.ws, self.rank, local = dist_env()
        if os.environ.get("GFS_BENCH_ONE_GPU") == "1":
            # test mode for the multi-rank path on a one-GPU box: every rank on cuda:0, gloo
            # (NCCL refuses two ranks on one GPU); never used for reported numbers
            local = 0
            if self.ws > 1:
                dist.init_process_group("gloo")
        elif self.ws > 1:
            dist.init_process_group("nccl", device_id=torch.device(f"cuda:{local}"))
        torch.cuda.set_device(local)
        self.local = local
        self.dev = f"cuda:{local}"
        g.build.build()
        self.hbm, self.hbm_src = peaks()
        self.stream = torch.cuda.Stream(device=self.dev)
        self.nproc = os.cpu_count() or 1

    def barrier(self):
        if self.ws > 1:
            self.dist.barrier()

    def allmax(self, x):
        t = self.torch.tensor([float(x)], device=self.dev, dtype=self.torch.float64)
        if self.ws > 1:
            self.dist.all_reduce(t, op=self.dist.ReduceOp.MAX)
        return float(t.item())

    def allmin(self, x):
        t = self.torch.tensor([float(x)], device=self.dev, dtype=self.torch.float64)
        if self.ws > 1:
            self.dist.all_reduce(t, op=self.dist.ReduceOp.MIN)
        return float(t.item())

    def allsum(self, x):
        t = self.torch.tensor([float(x)], device=self.dev, dtype=self.torch.float64)
        if self.ws > 1:
            self.dist.all_reduce(t)
        return float(t.item())

    def gather(self, obj):
        """Objects of every rank, on every rank (small: checksums, flags)."""
        if self.ws == 1:
            return [obj]
        out = [None] * self.ws
        self.dist.all_gather_object(out, obj)
        return out

    def shared_input(self, make):
        """A read-only input every rank uses: rank 0 writes it first, the others wait, then reuse it."""
        if self.rank == 0:
            r = make()
        self.barrier()
        if self.rank != 0:
            r = make()  # generators return at once when the file (and its marker) exists
        return r

    def timed(self, fn, reps):
        """Device time of each call on the bench stream (ms)."""
        torch, s = self.torch, self.stream
        ts = []
        for _ in range(reps):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            with torch.cuda.stream(s):
                e0.record(s)
                fn()
                e1.record(s)
            s.synchronize()
            ts.append(e0.elapsed_time(e1))
        return ts


# ---------------------------------------------------------------------- reference arm
def run_reference(args):
    """The CPU oracle as it stands (pread + position checksum) on the host cores, bounded sample."""
    ws, rank, _ = dist_env()
    if ws > 1 and rank != 0:
        return
    import gen
    import oracle
    size = args.file_gib << 30
    path = gen.splitmix_file(f"{SHM}/gfs_bench_c2_{size}_0.bin", size, seed=1000)
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
    val = gbs(sample, ms)
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


# ---------------------------------------------------------------------- C2 (headline)
def c2_phase(X):
    """The headline sweep: two files of file_gib each, swept alternately with a
    cache of cache_gib, so every page of every step is a miss."""
    args, torch, g, gen = X.args, X.torch, X.g, X.gen
    import oracle
    size = args.file_gib << 30
    P = args.page_kib << 10
    paths = [X.shared_input(lambda k=k: gen.splitmix_file(f"{SHM}/gfs_bench_c2_{size}_{k}.bin", size, seed=1000 + k))
             for k in range(2)]
    # the oracle's checksum of each file (rank 0, threaded), the expected value of every sweep
    want = [None, None]
    if X.rank == 0:
        t0 = time.perf_counter()
        want = [oracle.checksum_mt(p, 0, size) for p in paths]
        oracle_s = time.perf_counter() - t0
    else:
        oracle_s = 0.0
    want = X.gather(want)[0]
    h2d, h2d_ce, h2d_sm = pinned_h2d_gbs(torch, X.dev)
    X.barrier()
    h2d_conc = pinned_h2d_gbs(torch, X.dev)[0] if X.ws > 1 else h2d  # all ranks copy at once
    res = {"h2d_alone_GBps": round(h2d, 3), "h2d_copy_engine_GBps": round(h2d_ce, 3),
           "h2d_sm_pull_GBps": round(h2d_sm, 3), "h2d_concurrent_GBps": round(h2d_conc, 3)}
    fs = g.GpuFS(cache_bytes=args.cache_gib << 30, page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                 max_batch=1, timeout_ms=args.timeout_ms)
    grid = args.grid
    stream = X.stream
    scratch = torch.empty(grid * P, dtype=torch.uint8, device=X.dev)
    out = torch.zeros(2, dtype=torch.int64, device=X.dev)
    nstep = [0]
    sums = {}

    def step(mmap=False):
        out.zero_()
        fs.seqread(paths[nstep[0] % 2], size, P, grid=grid, stream=stream, sync=False, scratch=scratch, out=out,
                   use_mmap=mmap)
        nstep[0] += 1

    def check(label):
        stream.synchronize()
        v = out.cpu().numpy()
        if v[1] != 0:
            print("stats", fs.stats(), fs.host_stats(), fs.info(), file=sys.stderr)
            raise SystemExit(f"{label} sweep error {v[1]}")
        k = (nstep[0] - 1) % 2
        sums.setdefault(label, []).append(int(v[0]) & M64 == want[k])

    with torch.cuda.stream(stream):
        for _ in range(args.warmup):
            step()
            check("gread")
    fs.stats(reset=True)
    X.barrier()
    torch.cuda.synchronize()
    evs = []
    with Clocks(X.local) as clk:
        with torch.cuda.stream(stream):
            for _ in range(args.steps):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                step()
                e1.record(stream)
                evs.append((e0, e1))
            stream.synchronize()
    torch.cuda.synchronize()
    step_ms = [a.elapsed_time(b) for a, b in evs]
    ms_mean, ms_std = mstd(step_ms)
    checksum = int(out[0].item()) & M64
    sums["gread"].append(checksum == want[(nstep[0] - 1) % 2])
    st = fs.stats()
    hst = fs.host_stats()
    # e2e: the public API call with the host-side result read, wall clock
    res_h = torch.empty(2, dtype=torch.int64).pin_memory()
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    with torch.cuda.stream(stream):
        for _ in range(args.steps):
            step()
            stream.synchronize()
            res_h.copy_(out, non_blocking=True)  # D2H of the step's result (checksum, error)
            stream.synchronize()
            sums["gread"].append(int(res_h[0]) & M64 == want[(nstep[0] - 1) % 2])
    e2e_s = (time.perf_counter() - t0) / args.steps
    if int(res_h[1]) != 0:
        raise SystemExit(f"gread sweep error {int(res_h[1])}")
    # K1: the same sweep through gmmap/gmunmap
    if not args.no_k1:
        kt = []
        for _ in range(3):
            kt += X.timed(lambda: step(mmap=True), 1)
            check("gmmap")
        m, sd = mstd(kt[1:])
        res["k1_gmmap"] = {"GBps": round(gbs(size, m), 3), "frac_h2d": round(gbs(size, m) / h2d, 4),
                           "parity": all(sums.get("gmmap", [False]))}
    # zero-copy variant: both files registered, misses pull from the host page cache
    if not args.no_zc:
        try:
            t0 = time.perf_counter()
            modes = [fs.register_file(p_) for p_ in paths]
            reg_s = time.perf_counter() - t0
            fs.stats(reset=True)
            zt = []
            with torch.cuda.stream(stream):
                for r_ in range(args.warmup + args.steps):
                    t = X.timed(step, 1)
                    check("zc")
                    if r_ >= args.warmup:
                        zt += t
            zst = fs.stats()
            m, sd = mstd(zt)
            res["zero_copy"] = {"GBps": round(gbs(size, m), 3), "stddev": round(gbs(size, m) * sd / m, 3),
                                "frac_h2d": round(gbs(size, m) / h2d, 4), "register_s": round(reg_s, 2),
                                "registered_read_only": all(x == 1 for x in modes),
                                "zc_fill": zst["zc_fill"], "rpc_read": zst["rpc_read"],
                                "path_used": zst["zc_fill"] > 0 and zst["rpc_read"] == 0,
                                "parity": all(sums.get("zc", [False]))}
        except Exception as e:  # registration refused on this host: say so, keep the RPC headline
            res["zero_copy"] = {"unavailable": str(e)[:200]}
    fs.close()
    del scratch
    gb = gbs(size, ms_mean)
    res.update({"ms": round(ms_mean, 3), "ms_std": round(ms_std, 3), "GBps": round(gb, 3),
                "GBps_std": round(gb * ms_std / ms_mean, 3), "step_ms": [round(x, 3) for x in step_ms],
                "e2e_GBps": round(size / e2e_s / 1e9, 3), "checksum": hex(checksum),
                "parity": {"oracle_checksum_every_step": all(sums["gread"]), "oracle_s": round(oracle_s, 2),
                           "steps_checked": len(sums["gread"])},
                "counters": {k: st[k] for k in ("miss", "hit", "evict", "rpc", "timeout", "enomem", "ring_wait",
                                                "bytes_h2d")},
                "host": {"pread_GBps_per_thread": round(hst["bytes_h2d"] / max(hst["pread_ns"], 1), 3)
                         if hst["pread_ns"] else None},
                "clocks": clk.summary(), "h2d": h2d, "size": size, "paths": paths, "want": want})
    return res


def c2_split_phase(X, paths, size, want):
    """§8(e) C2 multi-GPU variant: byte ranges of ONE file, one per rank (strong
    scaling), checksums all-reduced (NCCL); parity vs the oracle's whole-file checksum."""
    args, torch, g = X.args, X.torch, X.g
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    P = args.page_kib << 10
    off, n = gdist.byte_range(size, X.ws, X.rank, P)
    with g.GpuFS(cache_bytes=args.cache_gib << 30, page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                 max_batch=1, timeout_ms=args.timeout_ms) as fs:
        scratch = torch.empty(args.grid * P, dtype=torch.uint8, device=X.dev)
        out = torch.zeros(2, dtype=torch.int64, device=X.dev)
        X.barrier()
        ts = X.timed(lambda: (out.zero_(), fs.seqread(paths[0], n, P, file_off=off, grid=args.grid,
                                                      stream=X.stream, sync=False, scratch=scratch, out=out)), 1)
        v = out.cpu().numpy()
    cs = torch.tensor([int(v[0])], dtype=torch.int64, device=X.dev)
    if X.ws > 1:
        X.dist.all_reduce(cs)  # the final reduction (NCCL): sum of the ranks' checksums mod 2^64
    ms = X.allmax(ts[0])
    return {"workload": f"one {size >> 30} GiB file split into {X.ws} byte ranges (strong scaling)",
            "GBps": round(gbs(size, ms), 3), "ms": round(ms, 3), "err": int(X.allmin(v[1])),
            "parity": (int(cs.item()) & M64) == want[0]}


# ---------------------------------------------------------------------- K4 (cache hit -> smem)
def hit_phase(X):
    """K4: 16 KiB greads into shared memory at random offsets of a warm file."""
    args, torch, g, gen = X.args, X.torch, X.g, X.gen
    import oracle
    P = args.hit_page_kib << 10
    size = args.hit_file_gib << 30
    path = X.shared_input(lambda: gen.splitmix_file(f"{SHM}/gfs_bench_hit_{size}.bin", size, seed=2000))
    chunk = 16384
    grid, calls = args.hit_grid, args.hit_calls
    rng = np.random.default_rng(7 + X.rank)
    offs = (rng.integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
    t0 = time.perf_counter()
    want = oracle.checksum_calls(path, offs, chunk, nthreads=X.nproc)
    oracle_s = time.perf_counter() - t0
    d_off = torch.as_tensor(offs.view(np.int64), device=X.dev)
    reps = args.reps
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=X.local,
                 daemon_threads=args.daemon_threads, timeout_ms=args.timeout_ms) as fs:
        s, err = fs.seqread(path, size, P, grid=296)  # pre-warm
        assert err == 0
        fs.stats(reset=True)
        out = torch.zeros(2, dtype=torch.int64, device=X.dev)
        raw = torch.empty(size, dtype=torch.uint8, device=X.dev)
        raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8), non_blocking=False)
        run_g = lambda: (out.zero_(), fs.randread(path, chunk, d_off, grid, block=args.hit_block,
                                                  stream=X.stream, sync=False, out=out))
        run_r = lambda: (out.zero_(), fs.randread(None, chunk, d_off, grid, block=args.hit_block, raw=raw,
                                                  stream=X.stream, sync=False, out=out))
        run_h = lambda: (out.zero_(), fs.randread(path, chunk, d_off, grid, block=args.hit_block, hint=True,
                                                  stream=X.stream, sync=False, out=out))
        X.timed(run_g, 2)
        X.timed(run_r, 2)
        X.timed(run_h, 2)
        X.barrier()
        tg = X.timed(run_g, reps)
        sg = int(out[0].item()) & M64
        tr = X.timed(run_r, reps)
        sr = int(out[0].item()) & M64
        th = X.timed(run_h, reps)
        sh = int(out[0].item()) & M64
        # K5 ablation (Table 2): every lookup under the file lock
        abl_calls = 32
        d_off_a = d_off[:grid * abl_calls]
        run_a = lambda: fs.randread(path, chunk, d_off_a, grid, block=args.hit_block, stream=X.stream, sync=False,
                                    out=out)
        run_a()
        ms_lockfree = float(np.median(X.timed(run_a, 3)))
        st = fs.stats()
        del raw
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                 timeout_ms=args.timeout_ms, flags=g.F_LOCKED_TRAVERSAL) as fl:
        s2, err2 = fl.seqread(path, size, P, grid=296)
        assert err2 == 0 and s2 == s
        run_l = lambda: fl.randread(path, chunk, d_off_a, grid, block=args.hit_block, stream=X.stream, sync=False,
                                    out=out)
        run_l()
        ms_locked = float(np.median(X.timed(run_l, 3)))
        stl = fl.stats()
    # ablation of the speculative one-page hit copy: the full K4 run with
    # every hit waiting for its reference before the copy starts
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                 timeout_ms=args.timeout_ms, flags=8) as fn:  # 8 = GFS_F_NO_SPECULATE
        s3, err3 = fn.seqread(path, size, P, grid=296)
        assert err3 == 0 and s3 == s
        run_n = lambda: (out.zero_(), fn.randread(path, chunk, d_off, grid, block=args.hit_block,
                                                  stream=X.stream, sync=False, out=out))
        X.timed(run_n, 2)
        tn = X.timed(run_n, reps)
        sn = int(out[0].item()) & M64
    nbytes = grid * calls * chunk
    mg, sdg = mstd(tg)
    mr, _ = mstd(tr)
    mh, sdh = mstd(th)
    mg_max = X.allmax(mg)
    gb = X.ws * gbs(nbytes, mg_max)
    return {"workload": f"K4: {grid} blocks x {calls} x 16 KiB gread -> smem, random offsets, {args.hit_file_gib} GiB "
                        f"warm file, {args.hit_page_kib} KiB pages, mean of {reps}",
            "GBps": round(gb, 3), "GBps_std": round(gb * sdg / mg, 3), "raw_GBps": round(gbs(nbytes, mr), 3),
            "vs_raw": round(mr / mg, 4), "ms": round(mg, 3),
            "roofline": {"bound": "hbm", "achieved": round(gbs(nbytes, mg), 3), "peak": X.hbm, "unit": "GB/s",
                         "frac": round(gbs(nbytes, mg) / X.hbm, 4), "traffic": None,
                         "note": "1 algorithmic HBM byte per delivered byte (frame read; destination is smem); per GPU"},
            "hint": {"GBps": round(X.ws * gbs(nbytes, X.allmax(mh)), 3), "vs_raw": round(mr / mh, 4),
                     "ms": round(mh, 3), "checksum_eq_oracle": sh == want,
                     "note": "gread_hint: each call names the block's next offset, whose leaf slot is read while "
                             "the current copy is in flight (no reference; the next call's speculative copy "
                             "starts without a tree access)"},
            "no_speculate": {"GBps": round(X.ws * gbs(nbytes, X.allmax(mstd(tn)[0])), 3),
                             "vs_raw": round(mr / mstd(tn)[0], 4), "checksum_eq_oracle": sn == want,
                             "note": "GFS_F_NO_SPECULATE: one-page hits wait for the reference before the copy"},
            "parity": {"checksum_eq_oracle": sg == want, "raw_eq_oracle": sr == want, "hint_eq_oracle": sh == want,
                       "no_speculate_eq_oracle": sn == want,
                       "oracle_s": round(oracle_s, 2)},
            "misses_after_warm": st["miss"],
            "k5_locked_ablation": {"calls_per_block": abl_calls, "lockfree_ms": round(ms_lockfree, 3),
                                   "locked_ms": round(ms_locked, 3),
                                   "lockfree_speedup": round(ms_locked / ms_lockfree, 2),
                                   "locked_lookups": stl["locked"],
                                   "note": "GFS_F_LOCKED_TRAVERSAL: every lookup takes the file lock (the paper "
                                           "reports lock-free ~3x faster, P:L1047-1048)"}}


# ---------------------------------------------------------------------- HG (cache hit -> global)
def hit_global_phase(X):
    """§8(a) a5: cache-hit gread of 256 KiB - 2 MiB chunks into global memory
    (P:L1023-1037 is the paper's hit experiment): a warm file swept into a
    destination of the file's size; 2 HBM bytes per delivered byte. Parity: the
    destination's position-weighted checksum == the oracle's over the file."""
    args, torch, g, gen = X.args, X.torch, X.g, X.gen
    import oracle
    size = args.hg_gib << 30
    P = 2 << 20
    path = X.shared_input(lambda: gen.splitmix_file(f"{SHM}/gfs_bench_hg_{size}.bin", size, seed=3000))
    want = oracle.checksum_mt(path, 0, size, nthreads=X.nproc) if X.rank == 0 else None
    want = X.gather(want)[0]
    points = []
    with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, device=X.local,
                 daemon_threads=args.daemon_threads, timeout_ms=args.timeout_ms) as fs:
        s, err = fs.seqread(path, size, P, grid=296)  # pre-warm
        assert err == 0
        fs.stats(reset=True)
        dst = torch.empty(size, dtype=torch.uint8, device=X.dev)
        out = torch.zeros(2, dtype=torch.int64, device=X.dev)
        for ck in (256 << 10, 1 << 20, 2 << 20):
            dst.zero_()
            run = lambda: fs.seqread(path, size, ck, grid=args.hg_grid, stream=X.stream, sync=False, scratch=dst,
                                     out=out, to_global=True)
            X.timed(run, 1)
            X.barrier()
            ts = X.timed(run, args.reps)
            err = int(out[1].item())
            # destination checksum on the device: sum_j w_j (2j + 1) mod 2^64 over 8-byte words
            cs = 0
            words = dst.view(torch.int64)
            step = 1 << 27
            for a in range(0, words.numel(), step):
                w_ = words[a:a + step]
                j = torch.arange(a, a + w_.numel(), device=X.dev, dtype=torch.int64)
                cs = (cs + int((w_ * (2 * j + 1)).sum().item())) & M64
            m, sd = mstd(ts)
            mm = X.allmax(m)
            points.append({"chunk_kib": ck >> 10, "GBps": round(X.ws * gbs(size, mm), 3),
                           "GBps_std": round(gbs(size, m) * sd / m, 3),
                           "frac_hbm_2B": round(2 * gbs(size, m) / X.hbm, 4), "err": err, "parity": cs == want})
        st = fs.stats()
        del dst
    best = max(points, key=lambda p: p["frac_hbm_2B"])
    return {"workload": f"warm {args.hg_gib} GiB file (2 MiB pages) swept into a {args.hg_gib} GiB device buffer, "
                        f"grid {args.hg_grid}x256, mean of {args.reps} per chunk size",
            "points": points, "misses_after_warm": st["miss"],
            "roofline": {"bound": "hbm", "achieved": round(best["frac_hbm_2B"] * X.hbm, 3), "peak": X.hbm,
                         "unit": "GB/s", "frac": best["frac_hbm_2B"],
                         "note": "2 HBM bytes per delivered byte (frame read + destination write), best chunk; per GPU"}}


# ---------------------------------------------------------------------- C3 mat-vec
def matvec_phase(X, h2d):
    """C3 (configs[2]): y = A x with A (rows x 131072 fp32) larger than the 2 GiB
    cache, read through gmmap, y through gwrite + gfsync. Every
    timed pass runs on a fresh cache (all misses). At N > 1 rank r computes the
    row block r (its own y shard file) and the shards are all-gathered (NCCL)."""
    args, torch, g, gen = X.args, X.torch, X.g, X.gen
    import oracle
    rows, cols = args.mv_rows, 131072
    m = X.shared_input(lambda: gen.matrix_files(f"{SHM}/gfs_bench_c3", rows, cols, seed=3))
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    r0, r1 = gdist.row_block(rows, X.ws, X.rank)
    nr = r1 - r0
    ypath = f"{SHM}/gfs_bench_c3/y_{X.rank}_{X.ws}.f32"
    nbytes = nr * cols * 4
    ts, link, errs, miss = [], [], [], []
    state = dict(x=torch.empty(cols, dtype=torch.float32, device=X.dev),
                 y=torch.empty(nr, dtype=torch.float32, device=X.dev),
                 err=torch.zeros(2, dtype=torch.int64, device=X.dev))
    for it in range(1 + args.mv_passes):  # pass 0: untimed warm-up of the process (not of the cache)
        with g.GpuFS(cache_bytes=2 << 30, page_size=2 << 20, device=X.local, daemon_threads=args.daemon_threads,
                     max_batch=1, timeout_ms=args.timeout_ms) as fs:
            X.barrier()
            t = X.timed(lambda: fs.matvec(m["A"], m["x"], ypath, rows, cols, stream=X.stream, sync=False,
                                          state=state, row0=r0, nrows=nr), 1)
            st = fs.stats()
            if it:
                ts += t
                link.append(st["bytes_h2d"])
                miss.append(st["miss"])
            errs.append(int(state["err"][0].item()))
    y = state["y"]
    # gather the y shards (NCCL all-gather of equal-size shards, zero-padded)
    yfull = gdist.gather_rows(X.dist.group.WORLD if X.ws > 1 else None, y[:nr], rows)
    yfull = yfull.cpu().numpy().astype(np.float64)
    ymine = y[:nr].cpu().numpy()
    yh = np.fromfile(ypath, dtype="<f4")
    ok_file = yh.size == nr and np.array_equal(yh, ymine)
    ok_file = X.allmin(1.0 if ok_file else 0.0) == 1.0
    mt, sdt = mstd(ts)
    mt_max = X.allmax(mt)
    gb = gbs(rows * cols * 4, mt_max)
    link_gbs = gbs(statistics.mean(link), mt)
    out = {"workload": f"C3: {rows} x {cols} fp32 matrix ({rows * cols * 4 >> 20} MiB) > 2 GiB cache, 2 MiB pages, "
                       f"gmmap rows, gwrite+gfsync y; fresh cache every pass, mean of {args.mv_passes}; "
                       f"{X.ws} row block(s), y all-gathered",
           "GBps": round(gb, 3), "GBps_std": round(gb * sdt / mt, 3), "ms": round(mt_max, 3),
           "err": min(errs), "misses_per_pass": miss, "link_bytes_per_pass": link,
           "roofline": {"bound": "h2d", "achieved": round(link_gbs, 3), "peak": round(h2d, 3), "unit": "GB/s",
                        "frac": round(link_gbs / h2d, 4),
                        "note": "host-link bytes the pass moved (bytes_h2d counter) over its time; per GPU"}}
    if X.rank == 0:
        t0 = time.perf_counter()
        ref = oracle.matvec(m["A"], m["x"], rows, cols, nthreads=X.nproc)
        dt = time.perf_counter() - t0
        rel = float(np.max(np.abs(yfull - ref) / np.maximum(np.abs(ref), 1e-300)))
        out["parity"] = {"rows_checked": int(rows), "max_rel_err": rel, "ok": rel <= 1e-5 and ok_file,
                         "y_file_eq_y": bool(ok_file)}
        out["cpu_baseline"] = {"value": round(gbs(rows * cols * 4, dt * 1e3), 3), "unit": "GB/s", "cores": X.nproc,
                               "kind": "oracle", "sample": f"all {rows} rows, float64, {X.nproc} threads"}
    # the same product with the matrix registered (zero-copy misses)
    if not args.no_zc and X.ws == 1:
        try:
            with g.GpuFS(cache_bytes=2 << 30, page_size=2 << 20, device=X.local, daemon_threads=args.daemon_threads,
                         max_batch=1, timeout_ms=args.timeout_ms) as fs:
                t0 = time.perf_counter()
                fs.register_file(m["A"])
                reg_s = time.perf_counter() - t0
                zt = X.timed(lambda: fs.matvec(m["A"], m["x"], ypath, rows, cols, stream=X.stream, sync=False,
                                               state=state), 1)
                zst = fs.stats()
                zy = state["y"].cpu().numpy()
            out["zero_copy"] = {"GBps": round(gbs(nbytes, zt[0]), 3), "frac_h2d": round(gbs(nbytes, zt[0]) / h2d, 4),
                                "register_s": round(reg_s, 2), "zc_fill": zst["zc_fill"], "rpc_read": zst["rpc_read"],
                                # every matrix page through the registered mapping; the only READ RPCs are
                                # the x vector's pages (x is not registered)
                                "path_used": (zst["zc_fill"] >= -(-nbytes // (2 << 20))
                                              and zst["rpc_read"] <= -(-cols * 4 // (2 << 20))),
                                "y_equal_rpc_path": bool(np.array_equal(zy, ymine))}
        except Exception as e:
            out["zero_copy"] = {"unavailable": str(e)[:200]}
    return out


# ---------------------------------------------------------------------- grep (C1, C4)
def grep_run(X, fs, d, lst, reps, hits, file_ids, chunk=16384, block=128):
    """cold (first run on fs) + warm runs (files kept open): device ms of each."""
    torch = X.torch
    state = fs.grep_state(d, lst, hits=hits, keep_open=True, rec_cap=1 << 24, pair_cap=1 << 23, chunk=chunk,
                          block=block, file_ids=file_ids)
    times = []
    for it in range(1 + reps):
        X.barrier()
        t = X.timed(lambda: fs.grep(d, lst, hits=hits, keep_open=True, stream=X.stream, sync=False, state=state,
                                    chunk=chunk, block=block), 1)
        times += t
    out = fs.grep(d, lst, hits=hits, keep_open=True, stream=X.stream, state=state, chunk=chunk, block=block)
    return times[0], times[1:], out, state


def grep_graph_run(X, fs, state, d, lst, reps, hits, chunk=16384, block=128):
    """The same warm run replayed from a CUDA graph (gfs_grep_graph_create): device ms
    of each replay and the last replay's output (checked against the oracle by the caller)."""
    fs.grep_graph(state, d, lst)
    run = lambda: fs.grep(d, lst, hits=hits, keep_open=True, stream=X.stream, sync=False, state=state, chunk=chunk,
                          block=block)
    X.timed(run, 1)
    X.barrier()
    t = X.timed(run, reps)
    out = fs.grep(d, lst, hits=hits, keep_open=True, stream=X.stream, state=state, chunk=chunk, block=block)
    fs.close_grep_graph(state)
    return t, out


def grep_parity(out, ref, hits):
    r = {"records": out["records"].tolist() == ref.records.tolist(),
         "totals": out["totals"].tolist() == ref.totals.tolist(),
         "digest": tuple(out["digest"]) == tuple(ref.digest), "err": out["summary"]["err"] == 0}
    if hits:
        r["hits"] = out["hits"].tolist() == ref.hits.tolist()
    return r


def c1_phase(X):
    """C1 (configs[0]): 64-word dictionary over 16 x 512 KiB; full parity incl. every hit."""
    args, g, gen = X.args, X.g, X.gen
    import oracle
    c = X.shared_input(lambda: gen.c1_corpus(f"{SHM}/gfs_bench_c1", seed=1))
    with g.GpuFS(cache_bytes=1 << 30, page_size=64 << 10, device=X.local, daemon_threads=args.daemon_threads,
                 timeout_ms=args.timeout_ms) as fs:
        cold, warm, out, state = grep_run(X, fs, c["dict"], c["list"], args.reps, True, None)
        tgr, out_g = grep_graph_run(X, fs, state, c["dict"], c["list"], args.reps, True)
    ref = oracle.grep(c["dict"], c["list"], want_hits=True, nthreads=X.nproc)
    nbytes = ref.bytes
    m, sd = mstd(warm)
    mg, sdg = mstd(tgr)
    return {"workload": "C1: 64-word dictionary, 16 x 512 KiB synthetic text, 64 KiB pages, cache > corpus",
            "cold_ms": round(cold, 3), "warm_ms": round(m, 3), "warm_ms_std": round(sd, 3),
            "warm_GBps": round(gbs(nbytes, m), 3), "nhits": int(out["digest"][2]),
            "warm_graph": {"ms": round(mg, 3), "ms_std": round(sdg, 3), "parity": grep_parity(out_g, ref, True),
                           "note": "the warm run replayed from a CUDA graph (gfs_grep_graph_create)"},
            "parity": {"records": out["records"].tolist() == ref.records.tolist(),
                       "totals": out["totals"].tolist() == ref.totals.tolist(),
                       "digest": tuple(out["digest"]) == tuple(ref.digest),
                       "hits": out["hits"].tolist() == ref.hits.tolist(), "err": out["summary"]["err"] == 0}}


def grep_phase(X):
    """C4 (configs[3]): grep -w of a 58k-word dictionary over a Linux-source-shaped
    tree, files sharded by LPT across ranks (global file ids); NCCL reduces totals
    and the digest, records are gathered to rank 0; the wall clock of the run
    includes that reduction."""
    args, torch, g, gen = X.args, X.torch, X.g, X.gen
    from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist
    root = f"{SHM}/gfs_bench_c4_{args.grep_files}_{args.grep_mib}"
    c = X.shared_input(lambda: gen.c4_corpus(root, seed=4, nfiles=args.grep_files, total_bytes=args.grep_mib << 20,
                                             nwords=58000))
    sizes = [os.path.getsize(p) for p in c["paths"]]  # metadata only, for the LPT split
    shard = gdist.lpt_shard(sizes, X.ws)[X.rank]
    lst = gdist.write_shard_list(c["paths"], shard, f"{root}/shard_{X.ws}_{X.rank}.txt")
    shard_bytes = int(sum(sizes[i] for i in shard))
    with g.GpuFS(cache_bytes=args.grep_cache_gib << 30, page_size=64 << 10, device=X.local,
                 daemon_threads=args.daemon_threads, max_files=1 << 16, timeout_ms=args.timeout_ms) as fs:
        cold, warm, out, _ = grep_run(X, fs, c["dict"], lst, args.reps, False, np.asarray(shard, np.uint32))
        gst = fs.stats()
        # wall clock of one more warm run including the final reduction: NCCL
        # all-reduce of the per-word totals and the digest on the device, the
        # raw records gathered to rank 0
        state = out["state"]
        nwords = out["summary"]["nwords"]
        X.barrier()
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        with torch.cuda.stream(X.stream):
            fs.grep(c["dict"], lst, hits=False, keep_open=True, stream=X.stream, sync=False, state=state)
            if X.ws > 1:
                X.dist.all_reduce(state["totals"][:nwords])
                sm_ = state["summary"][1:3].clone()  # nhits, digest sum (the xor is all-gathered)
                X.dist.all_reduce(sm_)
                xs = [torch.zeros(1, dtype=torch.int64, device=X.dev) for _ in range(X.ws)]
                X.dist.all_gather(xs, state["summary"][3:4].clone())
        X.stream.synchronize()
        if X.ws > 1:
            nrec = int(state["summary"][0].item())
            mine = state["rec"][:3 * nrec].cpu().numpy()
            objs = [None] * X.ws if X.rank == 0 else None
            X.dist.gather_object(mine, objs, dst=0)
        wall_ms = 1e3 * (time.perf_counter() - t0)
        tot, dig, allrecs = gdist.reduce_grep(X.dist.group.WORLD if X.ws > 1 else None, out["totals"],
                                              out["digest"], out["records"], device=torch.device(X.dev), root=0)
        tgr, out_g = grep_graph_run(X, fs, state, c["dict"], lst, args.reps, False) if X.ws == 1 else (None, None)
    cold_max = X.allmax(cold)
    m, sd = mstd(warm)
    m_max = X.allmax(m)
    total = args.grep_mib << 20
    res = {"workload": f"C4: {args.grep_files} files / {args.grep_mib} MiB C-like text, 58,000-word dictionary, "
                       f"LPT shard over {X.ws} GPU(s), 64 KiB pages; cold = fresh cache (OPEN + READ RPCs), "
                       f"warm = files kept open, pages cached; mean of {args.reps} warm runs",
           "cold": {"ms": round(cold_max, 3), "GBps": round(gbs(total, cold_max), 4),
                    "files_per_s": round(args.grep_files / (cold_max * 1e-3), 1)},
           "warm": {"ms": round(m_max, 3), "ms_std": round(sd, 3), "GBps": round(gbs(total, m_max), 4),
                    "files_per_s": round(args.grep_files / (m_max * 1e-3), 1)},
           "wall_with_reduce_ms": round(X.allmax(wall_ms), 3),
           "err": out["summary"]["err"], "nhits": int(dig[2]), "nrecords": int(len(allrecs)) if X.rank == 0 else None,
           "shard_bytes_rank0": shard_bytes, "rpc_open": gst["rpc_open"], "rpc_read": gst["rpc_read"],
           "misses": gst["miss"]}
    warm_gbs = gbs(total, m_max) / X.ws  # per GPU
    res["roofline_warm"] = {"bound": "hbm", "achieved": round(warm_gbs, 3), "peak": X.hbm, "unit": "GB/s",
                            "frac": round(warm_gbs / X.hbm, 5),
                            "note": "1 algorithmic HBM byte per corpus byte (frame -> smem); per GPU"}
    if X.rank == 0:
        import oracle
        t0 = time.perf_counter()
        ref = oracle.grep(c["dict"], c["list"], want_hits=False, nthreads=X.nproc)
        dt = time.perf_counter() - t0
        res["parity"] = {"totals": ref.totals.tolist() == list(map(int, tot)), "nhits": ref.digest[2] == int(dig[2]),
                         "records": ref.records.tolist() == allrecs.tolist(),
                         "digest": (ref.digest[0], ref.digest[1]) == (int(dig[0]), int(dig[1]))}
        res["cpu_baseline"] = {"value": round(ref.bytes / dt / 1e9, 4), "unit": "GB/s", "cores": X.nproc,
                               "kind": "oracle", "sample": f"whole C4 corpus ({ref.bytes} B), {X.nproc} threads"}
        if out_g is not None:
            mg, sdg = mstd(tgr)
            res["warm_graph"] = {"ms": round(mg, 3), "ms_std": round(sdg, 3), "parity": grep_parity(out_g, ref, False),
                                 "note": "the warm run replayed from a CUDA graph (gfs_grep_graph_create)"}
    return res


# ---------------------------------------------------------------------- Fig. 4
def fig4_phase(X, paths, size, h2d):
    """Fig. 4 analogue: miss-fill GB/s of a sequential gread sweep
    against page size. Sweeps alternate between the first 4 GiB of the two C2
    files with a 2 GiB cache, so every page is a miss (no LRU retention)."""
    args, torch, g = X.args, X.torch, X.g
    import oracle
    total = min(size, 4 << 30)
    want = [oracle.checksum_mt(p, 0, total, nthreads=X.nproc) for p in paths] if X.rank == 0 else None
    want = X.gather(want)[0]
    out = []
    for pk in (64, 256, 1024, 2048, 4096, 16384):
        P = pk << 10
        frames = (2 << 30) // P
        grid = int(min(296, frames // 2))
        with g.GpuFS(cache_bytes=2 << 30, page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                     timeout_ms=args.timeout_ms, max_batch=min(32, max(1, (8 << 20) // P))) as fs:
            chunk = max(P, 2 << 20)
            scratch = torch.empty(grid * chunk, dtype=torch.uint8, device=X.dev)
            res = torch.zeros(2, dtype=torch.int64, device=X.dev)
            ts, ok = [], True
            for rep in range(1 + args.fig4_reps):
                t = X.timed(lambda: (res.zero_(), fs.seqread(paths[rep % 2], total, chunk, grid=grid,
                                                             stream=X.stream, sync=False, scratch=scratch,
                                                             out=res)), 1)
                ok &= (int(res[0].item()) & M64) == want[rep % 2] and int(res[1].item()) == 0
                if rep:
                    ts += t
            st = fs.stats()
        m, sd = mstd(ts)
        out.append({"page_kib": pk, "GBps": round(gbs(total, m), 3), "GBps_std": round(gbs(total, m) * sd / m, 3),
                    "frac_h2d": round(gbs(total, m) / h2d, 4), "grid": grid, "misses": st["miss"],
                    "hits": st["hit"], "parity": bool(ok)})
    return {"workload": f"sequential gread sweep of {total >> 30} GiB, 2 GiB cache, chunk max(P, 2 MiB), "
                        f"mean of {args.fig4_reps}", "points": out}


# ---------------------------------------------------------------------- NEXT-2 read-ahead
def readahead_phase(X, paths, h2d):
    """NEXT-2: a sequential sweep by few blocks (each block's misses
    are serialised RPC -> host copy -> pull) with and without read-ahead (the next
    pages' READ RPCs posted, not waited for, and taken over by the later calls).
    The first 2 GiB of the two C2 files alternate under a 1 GiB cache: every page
    a miss. Parity: checksums == the oracle's."""
    args, torch, g = X.args, X.torch, X.g
    import oracle
    total, P = 2 << 30, 2 << 20
    want = [oracle.checksum_mt(p, 0, total, nthreads=X.nproc) for p in paths] if X.rank == 0 else None
    want = X.gather(want)[0]
    pts = []
    for grid in (8, 32):
        row = {"grid": grid}
        for ra in (0, 2):
            with g.GpuFS(cache_bytes=1 << 30, page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                         timeout_ms=args.timeout_ms, max_batch=1, readahead=ra) as fs:
                scratch = torch.empty(grid * P, dtype=torch.uint8, device=X.dev)
                res = torch.zeros(2, dtype=torch.int64, device=X.dev)
                ts, ok = [], True
                for rep in range(1 + args.reps):
                    t = X.timed(lambda: (res.zero_(), fs.seqread(paths[rep % 2], total, P, grid=grid,
                                                                 stream=X.stream, sync=False, scratch=scratch,
                                                                 out=res)), 1)
                    ok &= (int(res[0].item()) & M64) == want[rep % 2] and int(res[1].item()) == 0
                    if rep:
                        ts += t
                st = fs.stats()
            m, sd = mstd(ts)
            row[f"ra{ra}"] = {"GBps": round(gbs(total, m), 3), "GBps_std": round(gbs(total, m) * sd / m, 3),
                              "frac_h2d": round(gbs(total, m) / h2d, 4), "parity": bool(ok),
                              "ra_issued": st["ra_issued"], "ra_adopted": st["ra_adopted"],
                              "ra_reaped": st["ra_reaped"]}
        row["speedup"] = round(row["ra2"]["GBps"] / row["ra0"]["GBps"], 3)
        pts.append(row)
    return {"workload": f"sequential gread sweep of 2 GiB by 8 / 32 blocks, 2 MiB pages, 1 GiB cache, every page "
                        f"a miss; read-ahead 0 vs 2 pages; mean of {args.reps}", "points": pts}


# ---------------------------------------------------------------------- C5
def c5_phase(X, h2d):
    """C5 (configs[4]): repeated gwrite/gfsync then re-read across kernel launches.
    Rank r writes f_r (O_GWRONCE, new content every iteration) and gfsyncs it;
    after a barrier it re-reads f_{(r+1) % N} twice through its own cache: the
    first pass re-validates (close-to-open) and misses (or fills from
    the writer's cache over NVLink at N > 1), the second hits. Parity: the host
    file equals the source bytes and both re-read checksums equal the oracle's."""
    args, torch, g = X.args, X.torch, X.g
    import oracle
    P = 2 << 20
    size = args.c5_mib << 20
    root = f"{SHM}/gfs_bench_c5"
    os.makedirs(root, exist_ok=True)
    ws, rank = X.ws, X.rank
    mine, peer = f"{root}/f_{rank}.bin", f"{root}/f_{(rank + 1) % ws}.bin"
    if os.path.exists(mine):  # a write-once open does not truncate (R25): start from no file
        os.remove(mine)
    base = torch.from_numpy(np.random.default_rng(500 + rank).integers(0, 256, size=size, dtype=np.uint8)).to(X.dev)
    src = torch.empty_like(base)
    grid = 296
    times = {"write": [], "read_miss": [], "read_hit": []}
    ok_host, ok_read, errs = True, True, []
    stream = X.stream
    with g.GpuFS(cache_bytes=4 << 30, page_size=P, device=X.local, daemon_threads=args.daemon_threads,
                 max_batch=8, timeout_ms=args.timeout_ms, staging_slots=256) as fs:
        scratch = torch.empty(grid * P, dtype=torch.uint8, device=X.dev)
        out = torch.zeros(2, dtype=torch.int64, device=X.dev)
        wout = torch.zeros(2, dtype=torch.int64, device=X.dev)
        npeers, peer_err = 0, None
        if ws > 1 and not args.no_peers:
            # NEXT-1: every cache maps the others (CUDA IPC over NVLink)
            descs = [None] * ws
            try:
                mine_desc = fs.export()
            except Exception as e:
                mine_desc, peer_err = None, f"export: {e}"
            X.dist.all_gather_object(descs, mine_desc)
            for r, d in enumerate(descs):
                if r != rank and d is not None:
                    try:
                        fs.attach_peer(d)
                        npeers += 1
                    except Exception as e:
                        peer_err = f"attach rank {r}: {e}"
            if X.allmin(1 if npeers == ws - 1 else 0) == 0 and peer_err is None:
                peer_err = "some ranks could not attach every peer (results stay exact: peer fill is optional)"
        for it in range(args.c5_iters + 1):  # iteration 0 is untimed: it creates the files (tmpfs allocation)
            src.copy_(base)
            src.add_(it + 1)  # new content every iteration (mod 256), prepared before the timed region
            torch.cuda.synchronize()
            tw = X.timed(lambda: fs.seqwrite(mine, src, chunk=P, grid=grid, sync_grid=args.c5_sync_grid,
                                             stream=stream, sync=False, out=wout), 1)
            errs.append(int(wout[0].item()))
            X.barrier()  # every writer has gfsync'ed before anyone re-opens
            tm = X.timed(lambda: (out.zero_(), fs.seqread(peer, size, P, grid=grid, stream=stream, sync=False,
                                                          scratch=scratch, out=out)), 1)
            s1, err1 = int(out[0].item()) & M64, int(out[1].item())
            th = X.timed(lambda: (out.zero_(), fs.seqread(peer, size, P, grid=grid, stream=stream, sync=False,
                                                          scratch=scratch, out=out)), 1)
            s2, err2 = int(out[0].item()) & M64, int(out[1].item())
            errs += [err1, err2]
            if it:
                times["write"] += tw
                times["read_miss"] += tm
                times["read_hit"] += th
            want = oracle.checksum_mt(peer, 0, size, nthreads=X.nproc)
            ok_read &= s1 == want and s2 == want
            if it == args.c5_iters:
                hb = np.fromfile(mine, dtype=np.uint8)
                ok_host &= hb.size == size and np.array_equal(hb, src.cpu().numpy())
            X.barrier()  # nobody rewrites its file while a peer still reads it
        st = fs.stats()
        local_peer = None
        if ws == 1 and not args.no_peers:
            local_peer = c5_local_peer(X, fs, mine, size, P, grid, scratch, out)
    res = {}
    for k, v in times.items():
        m, sd = mstd(v)
        ms = X.allmax(m)
        res[k] = {"ms": round(ms, 3), "ms_std": round(sd, 3), "GBps": round(ws * gbs(size, ms), 3)}
    res.update({
        "workload": f"C5: {args.c5_iters} timed iterations (after one untimed) x (gwrite {args.c5_mib} MiB O_GWRONCE + gfsync from "
                    f"{args.c5_sync_grid} block(s); barrier; re-read the peer's file twice), 2 MiB pages, 4 GiB "
                    f"cache, {ws} GPU(s)",
        "err": min(errs) if errs else 0,
        "parity": {"host_file": bool(X.allmin(1 if ok_host else 0)), "reread_checksums": bool(X.allmin(1 if ok_read else 0))},
        "counters": {k: st[k] for k in ("miss", "hit", "writeback", "invalidate", "reopen_valid", "rpc_write",
                                        "rpc_read", "peer_fill", "bytes_peer")},
        "peers_attached": npeers,
        "peer_error": peer_err,
        "roofline": {"read_miss": ({"bound": "h2d", "peak": round(h2d, 3),
                                    "frac": round(res["read_miss"]["GBps"] / ws / h2d, 4)} if not npeers else
                                   {"bound": "nvlink", "peak": 900.0, "unit": "GB/s",
                                    "peak_source": "nominal NVLink 5 per-direction bandwidth per GPU",
                                    "frac": round(res["read_miss"]["GBps"] / ws / 900.0, 4)}),
                     "read_hit": {"bound": "hbm", "peak": X.hbm, "note": "2 B HBM per byte (frame read + copy out)",
                                  "frac": round(2 * res["read_hit"]["GBps"] / ws / X.hbm, 4)}},
    })
    if local_peer:
        res["read_peer_same_gpu"] = local_peer
    if ws == 1 and not args.no_rdwr:
        res["rdwr_shared_pages"] = rdwr_phase(X)
    return res


def rdwr_phase(X):
    """NEXT-4: two caches (stand-ins for two GPUs) open one existing
    file O_RDWR and write interleaved 64 KiB blocks of every 2 MiB page (false
    sharing), then gfsync: each write-back sends only the bytes that differ from
    the page's pristine copy, so both halves survive. Parity: the host file
    equals the original with both writers' blocks laid over it."""
    args, torch, g = X.args, X.torch, X.g
    P, blk = 2 << 20, 64 << 10
    size = args.rdwr_mib << 20
    root = f"{SHM}/gfs_bench_rdwr"
    os.makedirs(root, exist_ok=True)
    path = f"{root}/shared.bin"
    orig = np.random.default_rng(900).integers(0, 256, size=size, dtype=np.uint8)
    orig.tofile(path)
    offs = np.arange(0, size, blk, dtype=np.uint64)
    new = np.random.default_rng(901).integers(0, 256, size=size, dtype=np.uint8)
    times = {"gwrite": [], "gfsync": []}
    # 512 staging slots (1 GiB pinned): every O_RDWR page fetch holds one while its block pulls it
    caches = [g.GpuFS(cache_bytes=2 * size + (256 << 20), page_size=P, device=X.local,
                      daemon_threads=args.daemon_threads, max_batch=8, timeout_ms=args.timeout_ms,
                      staging_slots=512)
              for _ in range(2)]
    try:
        fds = [c.pin(path, flags=g.O_RDWR) for c in caches]
        for k, c in enumerate(caches):
            mine = offs[k::2]
            data = torch.from_numpy(np.concatenate([new[int(o):int(o) + blk] for o in mine])).to(X.dev)
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
            "gwrite_GBps": round(gbs(half, float(np.mean(times["gwrite"]))), 3),
            "gfsync_GBps": round(gbs(half, float(np.mean(times["gfsync"]))), 3),
            "parity": bool(ok), "writebacks": [x["writeback"] for x in st], "misses": [x["miss"] for x in st]}


def c5_local_peer(X, fs, path, size, P, grid, scratch, out):
    """N = 1 stand-in for NEXT-1 (peer-cache fill): a second cache on the same GPU
    attaches `fs` as its peer and reads the file `fs` holds (HBM -> HBM here;
    over NVLink between GPUs). Parity: the checksum equals the oracle's."""
    import oracle
    g = X.g
    want = oracle.checksum_mt(path, 0, size, nthreads=X.nproc)
    times, ok, st = [], True, {}
    for rep in range(3):
        with g.GpuFS(cache_bytes=4 << 30, page_size=P, device=fs.device, daemon_threads=2, max_batch=8,
                     timeout_ms=X.args.timeout_ms) as B:
            B.attach_peer(fs.export())
            X.torch.cuda.synchronize()
            t = X.timed(lambda: (out.zero_(), B.seqread(path, size, P, grid=grid, stream=X.stream, sync=False,
                                                        scratch=scratch, out=out)), 1)
            ok &= (int(out[0].item()) & M64) == want and int(out[1].item()) == 0
            times += t
            st = B.stats()
    ms = float(np.median(times))
    return {"ms": round(ms, 3), "GBps": round(gbs(size, ms), 3), "parity": bool(ok),
            "peer_fill": st["peer_fill"], "bytes_peer": st["bytes_peer"], "rpc_read": st["rpc_read"],
            "note": "second cache on the same GPU attached as a peer (NEXT-1 protocol; the copy is HBM->HBM, "
                    "not NVLink); includes the reader's gopen (OPEN RPC)"}


def cpu_baseline(X, path, size):
    """The oracle's pread + checksum on the host cores: one thread and nproc threads."""
    import oracle
    sample = min(size, X.args.ref_sample_mib << 20)
    t0 = time.perf_counter()
    oracle.checksum(path, 0, sample)
    dt1 = time.perf_counter() - t0
    t0 = time.perf_counter()
    oracle.checksum_mt(path, 0, size, nthreads=X.nproc)
    dtn = time.perf_counter() - t0
    return {"value": round(gbs(sample, dt1 * 1e3), 3), "unit": "GB/s", "cores": 1, "kind": "oracle",
            "sample": f"oracle pread+checksum of the first {X.args.ref_sample_mib} MiB of the sweep file, 1 thread",
            "nproc": {"value": round(gbs(size, dtn * 1e3), 3), "cores": X.nproc,
                      "sample": f"the whole {size >> 30} GiB sweep file, {X.nproc} threads"}}


def tmpfs_info():
    try:
        u = shutil.disk_usage(SHM)
        return {"total_gib": round(u.total / (1 << 30), 1), "free_gib": round(u.free / (1 << 30), 1)}
    except Exception:
        return None


def run_ours(args):
    X = Ctx(args)
    torch = X.torch
    need_gib = 2 * args.file_gib + args.hit_file_gib + args.hg_gib + 6 + 1
    tm = tmpfs_info()
    if tm and X.rank == 0 and tm["free_gib"] < need_gib:
        # shrink the optional hit->global file first, then report
        args.hg_gib = max(1, int(args.hg_gib - (need_gib - tm["free_gib"])))
    c2 = c2_phase(X)
    h2d, size, paths, want = c2["h2d"], c2["size"], c2["paths"], c2["want"]
    extra = {}
    if X.ws > 1 and not args.no_split:
        extra["c2_byte_split"] = c2_split_phase(X, paths, size, want)
    if not args.no_hit:
        extra["hit"] = hit_phase(X)
    if not args.no_hitg:
        extra["hit_global"] = hit_global_phase(X)
    if not args.no_c1:
        extra["c1"] = c1_phase(X)
    if not args.no_grep:
        extra["grep"] = grep_phase(X)
    if not args.no_matvec:
        extra["matvec"] = matvec_phase(X, h2d)
    if not args.no_fig4:
        extra["fig4_page_sweep"] = fig4_phase(X, paths, size, h2d)
    if not args.no_ra:
        extra["readahead"] = readahead_phase(X, paths, h2d)
    if not args.no_c5:
        extra["c5"] = c5_phase(X, h2d)
    cpu = cpu_baseline(X, paths[0], size) if (X.rank == 0 and not args.no_cpu) else None
    ms_max = X.allmax(c2["ms"])
    parity_c2 = X.allmin(1 if c2["parity"]["oracle_checksum_every_step"] else 0) == 1
    value = X.ws * gbs(size, ms_max)
    e2e = X.allsum(c2["e2e_GBps"])
    if X.rank != 0:
        return
    achieved = c2["GBps"]
    line = {
        "metric": "gread GB/s (miss fill, sequential sweep > cache)",
        "value": round(value, 3), "unit": "GB/s", "n_gpus": X.ws, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": round(ms_max, 3), "higher_is_better": True, "scaling": "weak", "vs_baseline": None,
        "dtype": "u8", "data": "synthetic",
        "config": {"workload": f"C2: sequential gread sweep of a {args.file_gib} GiB splitmix file per GPU (two "
                               f"files swept alternately: every page a miss), {args.cache_gib} GiB GPU cache, "
                               f"{args.page_kib} KiB pages, grid {args.grid}x256, {args.daemon_threads} daemon "
                               f"threads; tmpfs; file > cache and > L2 (no flush needed)",
                   "page_kib": args.page_kib, "cache_gib": args.cache_gib, "file_gib": args.file_gib,
                   "tmpfs": tm, "inputs": "read-only inputs shared by all ranks (written once by rank 0)"},
        "roofline": {"bound": "h2d", "achieved": round(achieved, 3), "peak": round(h2d, 3), "unit": "GB/s",
                     "frac": round(achieved / h2d, 4), "traffic": None,
                     "peak_source": "host->device link, 256 MiB of pinned memory, best of 10 of the copy engine and "
                                    "of an SM-pull kernel (gfs_probe_h2d), measured in this run"},
        "e2e": {"value": round(e2e, 3), "unit": "GB/s", "h2d_bytes_per_step": size, "d2h_bytes_per_step": 16},
        "gpu_launches": args.steps,
        "clocks": c2["clocks"],
        "stddev": {"GBps": c2["GBps_std"], "ms": c2["ms_std"], "steps": args.steps},
        "parity": {"c2_oracle_checksum_every_step_all_ranks": parity_c2},
        "c2": {k: c2[k] for k in ("h2d_alone_GBps", "h2d_copy_engine_GBps", "h2d_sm_pull_GBps",
                                   "h2d_concurrent_GBps", "step_ms", "e2e_GBps", "checksum", "parity", "counters",
                                   "host") if k in c2},
    }
    for k in ("k1_gmmap", "zero_copy"):
        if k in c2:
            line["c2"][k] = c2[k]
    line.update(extra)
    if cpu:
        line["cpu_baseline"] = cpu
    line["summary"] = make_summary(line, c2, extra)
    print(json.dumps(line), flush=True)


def make_summary(line, c2, extra):
    """The compact view, printed LAST in the JSON line (the driver keeps the line's tail)."""
    s = {"c2_GBps": line["value"], "c2_std": c2["GBps_std"], "c2_frac_h2d": line["roofline"]["frac"],
         "c2_parity": line["parity"]["c2_oracle_checksum_every_step_all_ranks"]}
    zc = c2.get("zero_copy") or {}
    if "GBps" in zc:
        s.update({"zc_GBps": zc["GBps"], "zc_parity": zc["parity"] and zc["path_used"]})
    k1 = c2.get("k1_gmmap") or {}
    if k1:
        s.update({"k1_GBps": k1["GBps"], "k1_parity": k1["parity"]})
    if "c2_byte_split" in extra:
        s.update({"c2split_GBps": extra["c2_byte_split"]["GBps"], "c2split_parity": extra["c2_byte_split"]["parity"]})
    h = extra.get("hit")
    if h:
        s.update({"k4_GBps": h["GBps"], "k4_frac_hbm": h["roofline"]["frac"], "k4_vs_raw": h["vs_raw"],
                  "k4_parity": h["parity"]["checksum_eq_oracle"],
                  "k4_no_speculate_vs_raw": h.get("no_speculate", {}).get("vs_raw")})
    hg = extra.get("hit_global")
    if hg:
        best = max(hg["points"], key=lambda p: p["frac_hbm_2B"])
        s.update({"hitg_GBps": best["GBps"], "hitg_chunk_kib": best["chunk_kib"], "hitg_frac_hbm_2B": best["frac_hbm_2B"],
                  "hitg_parity": all(p["parity"] for p in hg["points"])})
    c1 = extra.get("c1")
    if c1:
        s.update({"c1_warm_ms": c1["warm_ms"], "c1_cold_ms": c1["cold_ms"], "c1_parity": all(c1["parity"].values()),
                  "c1_graph_ms": c1["warm_graph"]["ms"], "c1_graph_parity": all(c1["warm_graph"]["parity"].values())})
    gr = extra.get("grep")
    if gr:
        s.update({"c4_warm_ms": gr["warm"]["ms"], "c4_warm_std": gr["warm"]["ms_std"], "c4_cold_ms": gr["cold"]["ms"],
                  "c4_wall_reduce_ms": gr["wall_with_reduce_ms"], "c4_frac_hbm": gr["roofline_warm"]["frac"],
                  "c4_parity": all(gr.get("parity", {}).values()) if gr.get("parity") else None})
        if gr.get("warm_graph"):
            s.update({"c4_graph_ms": gr["warm_graph"]["ms"],
                      "c4_graph_parity": all(gr["warm_graph"]["parity"].values())})
    mv = extra.get("matvec")
    if mv:
        s.update({"c3_GBps": mv["GBps"], "c3_std": mv["GBps_std"], "c3_link_frac_h2d": mv["roofline"]["frac"],
                  "c3_parity": mv.get("parity", {}).get("ok")})
    f4 = extra.get("fig4_page_sweep")
    if f4:
        s["fig4_frac_h2d"] = {p["page_kib"]: p["frac_h2d"] for p in f4["points"]}
        s["fig4_parity"] = all(p["parity"] for p in f4["points"])
    ra = extra.get("readahead")
    if ra:
        s["ra_grid8_GBps"] = [ra["points"][0]["ra0"]["GBps"], ra["points"][0]["ra2"]["GBps"]]
        s["ra_parity"] = all(p[k]["parity"] for p in ra["points"] for k in ("ra0", "ra2"))
    c5 = extra.get("c5")
    if c5:
        s.update({"c5_write_GBps": c5["write"]["GBps"], "c5_reread_miss_GBps": c5["read_miss"]["GBps"],
                  "c5_reread_hit_GBps": c5["read_hit"]["GBps"], "c5_parity": all(c5["parity"].values())})
    return s


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
    ap.add_argument("--reps", type=int, default=5, help="timed repetitions of the secondary phases (mean, stddev)")
    ap.add_argument("--hit-file-gib", type=int, default=4)
    ap.add_argument("--hit-page-kib", type=int, default=512)
    ap.add_argument("--hit-grid", type=int, default=1480)   # 10 blocks/SM (the register limit at 96 threads):
    ap.add_argument("--hit-block", type=int, default=96)    # lookups of one block overlap copies of the others
                                                            # (tools/k4_occ.py: 96 x 10 measured best)
    ap.add_argument("--hit-calls", type=int, default=820)  # ~1.21 M calls in all (1184 x 1024 before)
    ap.add_argument("--hg-gib", type=int, default=16, help="hit->global file size (GiB)")
    ap.add_argument("--hg-grid", type=int, default=2368)  # 592: 0.850, 1184: 0.866, 2368: 0.885 of HBM (2 MiB)
    ap.add_argument("--ref-sample-mib", type=int, default=2048)
    ap.add_argument("--timeout-ms", type=int, default=60000)
    ap.add_argument("--no-hit", action="store_true")
    ap.add_argument("--no-hitg", action="store_true")
    ap.add_argument("--no-c1", action="store_true")
    ap.add_argument("--no-grep", action="store_true")
    ap.add_argument("--no-matvec", action="store_true")
    ap.add_argument("--no-c5", action="store_true")
    ap.add_argument("--no-fig4", action="store_true")
    ap.add_argument("--no-ra", action="store_true", help="skip the read-ahead (NEXT-2) phase")
    ap.add_argument("--no-k1", action="store_true")
    ap.add_argument("--no-split", action="store_true", help="skip the C2 byte-range split (N > 1)")
    ap.add_argument("--no-zc", action="store_true", help="skip the zero-copy (registered file) variants")
    ap.add_argument("--fig4-reps", type=int, default=3)
    ap.add_argument("--c5-mib", type=int, default=512)
    ap.add_argument("--c5-iters", type=int, default=3)
    ap.add_argument("--c5-sync-grid", type=int, default=128)  # gfsync blocks (8: 25, 32: 28, 128: 30 GB/s)
    ap.add_argument("--mv-rows", type=int, default=11200)  # 5.6 GB (Fig. 8's 5600 MB point x2)
    ap.add_argument("--mv-passes", type=int, default=3)
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
