#!/usr/bin/env python3
"""Median device time of one SpMV configuration (CUDA events, L2 flushed).
usage: time_one.py LABEL MATRIX KERNEL [ENV=VAL ...]  -> one JSON line"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
for kv in sys.argv[4:]:
    k, v = kv.split("=")
    os.environ[k] = v
import numpy as np
import torch

import gen
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

label, w, kern = sys.argv[1], sys.argv[2], sys.argv[3]
C = gen.powerlaw() if w == "parboil" else gen.stencil27(int(w[7:])) if w.startswith("stencil") else gen.makea(w)
dev = torch.device("cuda:0")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (C.rowptr, C.colidx, C.vals))
x = torch.from_numpy(gen.uniform(C.n, seed=1, f32=C.vals.dtype == np.float32)).to(dev)
y = torch.empty(C.m, dtype=va.dtype, device=dev)
M = sp.CSRMatrix(rp, ci, va, C.n, kernel=kern, l2_window=os.environ.get("TIME_L2W") == "1")
flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
for _ in range(3):
    M.spmv(x, y)
if os.environ.get("TIME_STEADY") == "1":  # back-to-back launches (inputs larger than L2), as bench us_avg
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(30):
        M.spmv(x, y)
    b.record()
    b.synchronize()
    ms = a.elapsed_time(b) / 30
    print(json.dumps({"label": label, "matrix": w, "kernel": M.info()["kernel_name"], "mode": "steady",
                      "us": round(ms * 1e3, 2), "gbs": round(C.bytes_per_spmv() / (ms / 1e3) / 1e9, 1)}), flush=True)
    sys.exit(0)
ts = []
for _ in range(30):
    flush.zero_()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    M.spmv(x, y)
    b.record()
    b.synchronize()
    ts.append(a.elapsed_time(b))
ms = statistics.median(ts)
print(json.dumps({"label": label, "matrix": w, "kernel": M.info()["kernel_name"], "us": round(ms * 1e3, 2),
                  "gbs": round(C.bytes_per_spmv() / (ms / 1e3) / 1e9, 1)}), flush=True)
