#!/usr/bin/env python3
"""Extract per-launch DRAM traffic (dram__bytes_read.sum + dram__bytes_write.sum)
from an ncu --set full report into profiles/spmv_traffic.json under KEY.
usage: ncu_traffic.py REPORT KEY"""
import csv
import io
import json
import os
import subprocess
import sys

rep, key = sys.argv[1], sys.argv[2]
out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
hdr, units = rows[0], rows[1]
u = dict(zip(hdr, units))
scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
vals = []
for r in rows[2:]:
    d = dict(zip(hdr, r))
    b = sum(float(d[k]) * scale[u[k]] for k in ("dram__bytes_read.sum", "dram__bytes_write.sum"))
    vals.append(b)
path = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "profiles", "spmv_traffic.json")
tj = json.load(open(path)) if os.path.exists(path) else {}
tj[key] = int(sum(vals) / len(vals))
json.dump(tj, open(path, "w"), indent=1, sort_keys=True)
print(key, tj[key])
