#!/usr/bin/env python3
"""Aggregate an ncu --metrics gpu__time_duration.sum launch list (CSV) per kernel."""
import collections
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
hdr, data = None, []
for r in rows:
    if 'Kernel Name' in r:
        hdr = r
        continue
    if hdr and len(r) == len(hdr):
        data.append(dict(zip(hdr, r)))
agg = collections.defaultdict(lambda: [0, 0.0])
for d in data:
    if d.get('Metric Name') != 'gpu__time_duration.sum':
        continue
    k = d['Kernel Name'].split('(')[0][:70]
    agg[k][0] += 1
    agg[k][1] += float(d['Metric Value'])
tot = sum(v[1] for v in agg.values())
print(f"# {sys.argv[1]}: per-kernel device time (ncu, serialised, cold caches: compare shares, not absolutes)")
for k, v in sorted(agg.items(), key=lambda x: -x[1][1]):
    print(f"{k:72s} n={v[0]:4d} total={v[1] / 1e3:9.1f} us avg={v[1] / v[0] / 1e3:8.2f} us share={100 * v[1] / tot:5.1f}%")
