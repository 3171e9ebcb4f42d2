#!/usr/bin/env python3
"""Median device time of the matrix-free 27-point stencil on an N^3 grid
(CUDA events, L2 flushed).  usage: time_stencil.py LABEL N [ENV=VAL ...]"""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
for kv in sys.argv[3:]:
    k, v = kv.split("=")
    os.environ[k] = v
import torch

import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

label, N = sys.argv[1], int(sys.argv[2])
dev = torch.device("cuda:0")
x = torch.rand(N ** 3, dtype=torch.float64, device=dev)
y = torch.empty_like(x)
flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
for _ in range(3):
    sp.stencil27_apply(N, N, N, x, y)
ts = []
for _ in range(20):
    flush.zero_()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    sp.stencil27_apply(N, N, N, x, y)
    b.record()
    b.synchronize()
    ts.append(a.elapsed_time(b))
ms = statistics.median(ts)
print(json.dumps({"label": label, "N": N, "env": sys.argv[3:], "us": round(ms * 1e3, 2),
                  "gbs_own": round(16 * N ** 3 / (ms / 1e3) / 1e9, 1)}), flush=True)
