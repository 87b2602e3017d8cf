"""Per-run kernel times from an ncu --metrics gpu__time_duration.sum CSV (runs split evenly)."""
import csv, sys
rows = list(csv.reader(open(sys.argv[1])))
runs = int(sys.argv[2]) if len(sys.argv) > 2 else 1
i = [k for k, r in enumerate(rows) if r and r[0] == 'ID'][0]
hdr = rows[i]
seq = []
for r in rows[i + 1:]:
    d = dict(zip(hdr, r))
    if d.get('Metric Name') != 'gpu__time_duration.sum':
        continue
    v = float(d['Metric Value'].replace(',', ''))
    u = d['Metric Unit']
    v = v / 1e3 if u == 'ns' else v * 1e3 if u == 'ms' else v
    seq.append((d['Kernel Name'].split('(')[0].replace('<unnamed>::', ''), v))
n = len(seq) // runs
for run in range(runs):
    part = seq[run * n:(run + 1) * n]
    print("run", run, "total us %.0f" % sum(v for _, v in part), " ".join(f"{k}:{v:.0f}" for k, v in part))
