"""Aggregate an ncu --metrics gpu__time_duration.sum CSV into a per-kernel table (markdown)."""
import collections, csv, sys

rows = list(csv.reader(open(sys.argv[1])))
i = [k for k, r in enumerate(rows) if r and r[0] == 'ID'][0]
hdr = rows[i]
tot = collections.OrderedDict()
for r in rows[i + 1:]:
    d = dict(zip(hdr, r))
    if d.get('Metric Name') != 'gpu__time_duration.sum':
        continue
    v = float(d['Metric Value'].replace(',', ''))
    u = d['Metric Unit']
    ms = v / 1e6 if u == 'ns' else v / 1e3 if u == 'us' else v if u == 'ms' else v * 1e3
    k = d['Kernel Name'].split('(')[0].replace('<unnamed>::', '')
    n, t = tot.get(k, (0, 0.0))
    tot[k] = (n + 1, t + ms)
s = sum(t for _, t in tot.values())
print("| kernel | launches | total ms | share |\n|---|---|---|---|")
for k, (n, t) in sorted(tot.items(), key=lambda kv: -kv[1][1]):
    if t / s >= 0.0005:
        print(f"| {k} | {n} | {t:.2f} | {100 * t / s:.1f} % |")
