"""C4 grep: cold + warm runs with the cache counters of each run (what the
scan's reads did: fast-path hits, slow-path lookups, busy, retries)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
nf = int(os.environ.get("C4_FILES", "30000")); mib = int(os.environ.get("C4_MIB", "500"))
chunk = int(os.environ.get("CHUNK", "16384"))
whole = int(os.environ.get("WHOLE", "0"))
block = int(os.environ.get("BLOCK", "256"))
pair = int(os.environ.get("PAIR", str(1 << 21)))
runs = int(os.environ.get("RUNS", "3"))
c = gen.c4_corpus(f"/dev/shm/gfs_bench_c4_{nf}_{mib}", seed=4, nfiles=nf, total_bytes=mib << 20, nwords=58000)
s = torch.cuda.Stream()
with g.GpuFS(cache_bytes=4 << 30, page_size=64 << 10, daemon_threads=12, max_files=1 << 16) as fs:
    state = fs.grep_state(c["dict"], c["list"], keep_open=True, rec_cap=1 << 24, chunk=chunk, whole_max=whole, pair_cap=pair, block=block)
    for it in range(runs):
        fs.stats(reset=True)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        with torch.cuda.stream(s):
            e0.record(s)
            state = fs.grep(c["dict"], c["list"], keep_open=True, rec_cap=1 << 24, stream=s, sync=False,
                            state=state, chunk=chunk, whole_max=whole, pair_cap=pair, block=block)
            e1.record(s)
        s.synchronize()
        summ = dict(zip(g.GREP_SUMMARY, (int(x) for x in state["summary"].cpu().numpy())))
        st = fs.stats()
        print("cold" if it == 0 else "warm", f"{e0.elapsed_time(e1):.3f} ms", summ, flush=True)
        print("   ", {k: v for k, v in st.items() if v}, flush=True)
