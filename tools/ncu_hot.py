"""Hot SASS lines of one kernel in an ncu report (stall samples, executed instructions).
usage: ncu_hot.py REPORT [N]"""
import csv, subprocess, sys
rep = sys.argv[1]
n = int(sys.argv[2]) if len(sys.argv) > 2 else 40
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"], capture_output=True,
                     text=True).stdout
r = list(csv.reader(out.splitlines()))
h = [i for i, x in enumerate(r) if "Source" in x and "# Samples" in x][0]
H = r[h]
si, src, ie = H.index("Warp Stall Sampling (All Samples)"), H.index("Source"), H.index("Instructions Executed")
rows = [x for x in r[h + 1:] if len(x) > si]
tot = sum(float(x[si] or 0) for x in rows)
ti = sum(float(x[ie] or 0) for x in rows)
print(f"samples {tot:.0f} warp-inst {ti:.0f} sass-lines {len(rows)}")
idx = sorted(range(len(rows)), key=lambda i: -float(rows[i][si] or 0))[:n]
for i in sorted(idx):
    x = rows[i]
    print(f"{i:6d} {float(x[si]) / tot * 100:5.1f}%  exec {float(x[ie] or 0):>10.0f}  {x[src].strip()[:90]}")
