"""Markdown table of a bench JSON line (profiles/r01_bench_full.json.log) for profiles/r01_summary.md."""
import json
import sys

d = json.loads(open(sys.argv[1]).read())
r = json.loads(open(sys.argv[2]).read()) if len(sys.argv) > 2 else None
g, mv, c5, h = d["grep"], d["matvec"], d["c5"], d["hit"]
z = d.get("c2_zero_copy", {})
print("| phase | result | roofline |\n|---|---|---|")
print(f"| C2 miss-fill sweep, RPC path (headline `value`) | {d['value']} GB/s (e2e {d['e2e']['value']}) | "
      f"{100 * d['roofline']['frac']:.1f} % of in-run pinned H2D ({d['roofline']['peak']} GB/s) |")
if "GBps" in z:
    print(f"| C2 sweep, zero-copy (registered files, no READ RPC) | {z['GBps']} GB/s, {z['zc_fill']} direct fills, "
          f"{z['rpc_read']} READ RPCs, checksums = RPC sweep: {z['checksum_matches_rpc_sweep']} (registration "
          f"{z['register_s']} s, setup) | {100 * z['frac_h2d']:.1f} % of H2D |")
print(f"| K1 gmmap variant of the sweep | {d['k1_gmmap']['GBps']} GB/s, checksum = gread sweep | "
      f"{100 * d['k1_gmmap']['frac_h2d']:.1f} % of H2D |")
print(f"| K4 cache-hit gread -> smem | {h['GBps']} GB/s (raw TMA kernel {h['raw_GBps']}) | "
      f"{100 * h['roofline']['frac']:.1f} % of measured HBM ({h['roofline']['peak']} GB/s) |")
k5 = h["k5_locked_ablation"]
print(f"| K5 ablation: every lookup under the file lock | {k5['locked_ms']} ms vs lock-free {k5['lockfree_ms']} ms "
      f"({k5['lockfree_speedup']}x) | — |")
print(f"| C3 out-of-core mat-vec | {mv['GBps']} GB/s | {100 * mv['roofline']['frac']:.1f} % of H2D |")
zm = mv.get("zero_copy", {})
if "GBps" in zm:
    print(f"| C3 with the matrix registered (zero-copy) | {zm['GBps']} GB/s, y identical: {zm['y_equal_rpc_path']} | "
          f"{100 * zm['frac_h2d']:.1f} % of H2D |")
print(f"| C4 grep, 30k files / 500 MiB | warm {g['warm']['ms']} ms ({g['warm']['GBps']} GB/s, "
      f"{g['warm']['files_per_s']:.0f} files/s); cold {g['cold']['ms']} ms | warm "
      f"{100 * g['roofline_warm']['frac']:.2f} % of HBM (per-item latency bound, DESIGN §6.1) |")
print(f"| C5 write + gfsync / re-read | write {c5['write']['GBps']} GB/s; re-read miss {c5['read_miss']['GBps']} GB/s, "
      f"hit {c5['read_hit']['GBps']} GB/s | miss {100 * c5['roofline']['read_miss']['frac']:.1f} % of H2D |")
lp = c5["read_peer_same_gpu"]
print(f"| NEXT-1 peer-cache re-read (2nd cache, same GPU) | {lp['GBps']} GB/s, {lp['peer_fill']} pages from the peer, "
      f"{lp['rpc_read']} host reads | HBM->HBM stand-in for NVLink |")
rw = c5["rdwr_shared_pages"]
print(f"| NEXT-4 O_RDWR shared pages (2 caches) | gwrite {rw['gwrite_GBps']} GB/s, diff write-back "
      f"{rw['gfsync_GBps']} GB/s, parity {rw['parity']} | — |")
pts = d["fig4_page_sweep"]["points"]
print("| Fig. 4 page-size sweep (4 GiB, 2 GiB cache, RPC path) | " +
      ", ".join(f"{p['page_kib']} KiB: {p['GBps']}" for p in pts) + " GB/s | " +
      ", ".join(f"{100 * p['frac_h2d']:.0f} %" for p in pts) + " of H2D |")
if r:
    print(f"| CPU oracle (reference arm) | {r['value']} {r['unit']} | {r['cpu_baseline']['sample']}, "
          f"{r['cpu_baseline']['cores']} core(s) |")
print(f"\nParity in the same run: grep {g['parity']}, mat-vec {mv['parity_ok']}, C5 {c5['parity']}. "
      f"Clocks: {d['clocks']}.")
