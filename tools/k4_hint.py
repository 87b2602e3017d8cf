"""K4 variants side by side (event-timed): plain gread, gread_hint, raw TMA; GRID/BLOCK/CALLS env."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import gen
import oracle
import paper_conf_asplos_silbersteinfkw13_b200 as g
size, P, chunk = int(os.environ.get("GIB", "4")) << 30, 512 << 10, 16384
only = os.environ.get("ONLY")
grid, block, calls = (int(os.environ.get(k, d)) for k, d in (("GRID", "1184"), ("BLOCK", "128"), ("CALLS", "256")))
path = gen.splitmix_file(f"/dev/shm/gfs_bench_hit_{size}.bin", size, seed=2000)
offs = (np.random.default_rng(7).integers(0, size // chunk, size=grid * calls) * chunk).astype(np.uint64)
want = oracle.checksum_calls(path, offs, chunk, nthreads=os.cpu_count())
with g.GpuFS(cache_bytes=size + (256 << 20), page_size=P, daemon_threads=12) as fs:
    assert fs.seqread(path, size, P, grid=296)[1] == 0
    fs.pin(path)  # held open: a profiled kernel's gopen needs no RPC (ncu replays kernels, not the host)
    d_off = torch.as_tensor(offs.view(np.int64), device="cuda:0")
    raw = torch.empty(size, dtype=torch.uint8, device="cuda:0")
    raw.copy_(torch.from_file(path, shared=False, size=size, dtype=torch.uint8))
    out = torch.zeros(2, dtype=torch.int64, device="cuda:0")
    s = torch.cuda.Stream()
    runs = {"gread": lambda: fs.randread(path, chunk, d_off, grid, block=block, stream=s, sync=False, out=out),
            "hint": lambda: fs.randread(path, chunk, d_off, grid, block=block, hint=True, stream=s, sync=False, out=out),
            "raw": lambda: fs.randread(None, chunk, d_off, grid, block=block, raw=raw, stream=s, sync=False, out=out)}
    nbytes = grid * calls * chunk
    res = {}
    for name, fn in runs.items():
        if only and name != only:
            continue
        ts = []
        fs.stats(reset=True)
        for it in range(7):
            out.zero_()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s); fn(); e1.record(s); s.synchronize()
            if it >= 2: ts.append(e0.elapsed_time(e1))
        ok = (int(out[0].item()) & ((1 << 64) - 1)) == want
        res[name] = np.mean(ts)
        st = fs.stats()
        print(f"{name:6s} {np.mean(ts):.3f} ms  {nbytes / np.mean(ts) / 1e6:.1f} GB/s  parity {ok}  "
              f"hits/call {st.get('hit', 0) / (7 * grid * calls):.3f}", flush=True)
    if not only:
        print("gread/raw", round(res["raw"] / res["gread"], 4), "hint/raw", round(res["raw"] / res["hint"], 4))
