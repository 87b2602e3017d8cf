"""Aggregate an ncu source page (SASS rows: stall samples, executed instructions)
by CUDA source line, using the line table of the same build's cubin.
usage: ncu_lines.py REPORT CUBIN KERNEL_SUBSTR [N]"""
import collections, csv, re, subprocess, sys
rep, cubin, kname = sys.argv[1], sys.argv[2], sys.argv[3]
n = int(sys.argv[4]) if len(sys.argv) > 4 else 50
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"], capture_output=True,
                     text=True).stdout
r = list(csv.reader(out.splitlines()))
h = [i for i, x in enumerate(r) if "Source" in x and "# Samples" in x][0]
H = r[h]
si, ie, src = H.index("Warp Stall Sampling (All Samples)"), H.index("Instructions Executed"), H.index("Source")
rows = [x for x in r[h + 1:] if len(x) > si]
dis = subprocess.run(["nvdisasm", "--print-line-info", cubin], capture_output=True, text=True).stdout.split("\n")
fn, cur, seq = None, None, []
for l in dis:
    m0 = re.match(r"\s*\.text\.(\S+):", l)
    if m0:
        fn = m0.group(1)
    m = re.search(r'## File "([^"]+)", line (\d+)', l)
    if m:
        cur = (m.group(1).split("/")[-1], int(m.group(2)))
    if fn and kname in fn and re.match(r"\s*/\*[0-9a-f]{4,}\*/", l):
        seq.append((cur, l.split("*/", 1)[1].strip()))
print(f"ncu rows {len(rows)}  cubin instructions {len(seq)}")
agg = collections.defaultdict(lambda: [0.0, 0.0])
ts = sum(float(x[si] or 0) for x in rows)
ti = sum(float(x[ie] or 0) for x in rows)
for i, x in enumerate(rows):
    k = seq[i][0] if i < len(seq) else ("?", 0)
    agg[k][0] += float(x[si] or 0)
    agg[k][1] += float(x[ie] or 0)
srcs = {}
def line(k):
    if k[0] not in srcs:
        try:
            import glob
            p = [q for q in glob.glob("**/" + k[0], recursive=True)][0]
            srcs[k[0]] = open(p).read().split("\n")
        except Exception:
            srcs[k[0]] = []
    L = srcs[k[0]]
    return L[k[1] - 1].strip()[:70] if 0 < k[1] <= len(L) else ""
for k, (sm, ex) in sorted(agg.items(), key=lambda kv: -kv[1][0])[:n]:
    print(f"{sm / ts * 100:5.1f}% samp {ex / ti * 100:5.1f}% inst  {k[0]}:{k[1]}  {line(k)}")
