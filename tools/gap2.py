#!/usr/bin/env python3
"""The bench's roofline leg in isolation, step by step, to see what moves the
graph-replayed SpMV time: replays printed one by one, optionally after the CG
steps (npb_outer) and with the nvidia-smi clock sampler running.
usage: gap2.py [--cg] [--smi] [--reps N]"""
import argparse
import os
import subprocess
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import json  # noqa: E402

import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--cg", action="store_true")
ap.add_argument("--smi", action="store_true")
ap.add_argument("--reps", type=int, default=10)
args = ap.parse_args()
dev = torch.device("cuda:0")
torch.cuda.set_stream(torch.cuda.Stream(dev))
stream = torch.cuda.current_stream(dev)
A = gen.makea("C")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
M = sp.CSRMatrix(rp, ci, va, A.n)
M.set_cg_variant("cgcg")
smi = None
if args.smi:
    smi = subprocess.Popen(["nvidia-smi", "-i", "0", "--query-gpu=clocks.sm", "--format=csv,noheader", "-lms", "50"],
                           stdout=subprocess.DEVNULL, stderr=subprocess.DEVNULL)
if args.cg:
    x = torch.ones(A.n, dtype=torch.float64, device=dev)
    z = torch.empty_like(x)
    o2 = torch.zeros(2, dtype=torch.float64, device=dev)
    for _ in range(13):
        M.npb_outer(x, z, 25, 110.0, o2)
    torch.cuda.synchronize()
p = torch.from_numpy(gen.uniform(A.n, seed=5)).to(dev)
q = torch.empty(A.n, dtype=torch.float64, device=dev)
for _ in range(3):
    M.spmv(p, q)
g = torch.cuda.CUDAGraph()
with torch.cuda.graph(g, stream=stream):
    for _ in range(args.reps):
        M.spmv(p, q)
g.replay()
torch.cuda.synchronize()
a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
ts = []
for _ in range(6):
    a.record(stream)
    g.replay()
    b.record(stream)
    b.synchronize()
    ts.append(round(a.elapsed_time(b) * 1e3 / args.reps, 2))
if smi:
    smi.terminate()
print(json.dumps({"cg": args.cg, "smi": args.smi, "reps": args.reps, "us": ts}), flush=True)
