"""C4 grep timing outside the bench: cold + N warm runs, device-timed with CUDA events."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
nf = int(os.environ.get("C4_FILES", "30000")); mib = int(os.environ.get("C4_MIB", "500"))
chunk = int(os.environ.get("CHUNK", "32768"))
block = int(os.environ.get("BLOCK", "256"))
runs = int(os.environ.get("RUNS", "6"))
c = gen.c4_corpus(f"/dev/shm/gfs_bench_c4_{nf}_{mib}", seed=4, nfiles=nf, total_bytes=mib << 20, nwords=58000)
s = torch.cuda.Stream()
with g.GpuFS(cache_bytes=4 << 30, page_size=64 << 10, daemon_threads=int(os.environ.get("DAEMON", "12")), max_files=1 << 16) as fs:
    state = fs.grep_state(c["dict"], c["list"], keep_open=True, rec_cap=1 << 24, chunk=chunk, block=block)
    for it in range(runs):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        with torch.cuda.stream(s):
            e0.record(s)
            state = fs.grep(c["dict"], c["list"], keep_open=True, rec_cap=1 << 24, stream=s,
                            sync=False, state=state, chunk=chunk, block=block)
            e1.record(s)
        s.synchronize()
        summ = dict(zip(g.GREP_SUMMARY, (int(x) for x in state["summary"].cpu().numpy())))
        if it == 0 and os.environ.get("HOST_STATS"):
            hs = fs.host_stats()
            print({k: hs[k] for k in ("open", "read", "open_ns", "open_sys_ns", "open_prefetch_ns", "open_table_ns", "open_vt_ns",
                                      "pread_ns", "busy_ns", "bytes_h2d")}, fs.stats()["rpc_open"], flush=True)
        print(f"chunk={chunk} block={block}", "cold" if it == 0 else "warm", f"{e0.elapsed_time(e1):.3f} ms",
              summ["err"], summ["nhits"], summ["nrecords"], summ["digest_xor"], flush=True)
