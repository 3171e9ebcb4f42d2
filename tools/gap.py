#!/usr/bin/env python3
"""Device time per XPLAN SpMV launch, back to back (CUDA events around 30
launches, eager and as a captured CUDA graph), to compare with the kernel span
the per-CTA globaltimer stamps give (tools/xplan_times.py): the difference is
the launch gap between consecutive kernels.  usage: gap.py CLASS [ones|rand]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import json  # noqa: E402

import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

cls = sys.argv[1]
xk = sys.argv[2] if len(sys.argv) > 2 else "ones"
dev = torch.device("cuda:0")
A = gen.makea(cls)
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
x = torch.ones(A.n, dtype=torch.float64, device=dev) if xk == "ones" else torch.from_numpy(gen.uniform(A.n, seed=1)).to(dev)
y = torch.empty(A.m, dtype=torch.float64, device=dev)
s = torch.cuda.Stream()
out = {"class": cls, "x": xk}
with torch.cuda.stream(s):
    M = sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan")  # the handle launches on the stream current at creation
    for _ in range(5):
        M.spmv(x, y)
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    for n in (1, 30):
        best = 1e9
        for _ in range(5):
            a.record(s)
            for _ in range(n):
                M.spmv(x, y)
            b.record(s)
            b.synchronize()
            best = min(best, a.elapsed_time(b) * 1e3 / n)
        out[f"eager_us_n{n}"] = round(best, 2)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        for _ in range(30):
            M.spmv(x, y)
    g.replay()
    best = 1e9
    for _ in range(5):
        a.record(s)
        g.replay()
        b.record(s)
        b.synchronize()
        best = min(best, a.elapsed_time(b) * 1e3 / 30)
    out["graph_us"] = round(best, 2)
print(json.dumps(out), flush=True)
