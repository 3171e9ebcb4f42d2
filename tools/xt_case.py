#!/usr/bin/env python3
"""One SpMV through the XT kernel on a named matrix, checked against the oracle.
usage: xt_case.py MATRIX [ENV=VAL ...]   MATRIX: powerlaw_small | laplace | S | W | A | B | C"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
for kv in sys.argv[2:]:
    k, v = kv.split("=")
    os.environ[k] = v
import numpy as np
import torch

import gen
import oracle
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

w = sys.argv[1]
A = (gen.powerlaw(m=20000, lmax=3000.0, beta=0.6, seed=5, f32=False) if w == "powerlaw_small"
     else gen.laplace1d(100001) if w == "laplace" else gen.makea(w))
dev = torch.device("cuda:0")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
xh = gen.uniform(A.n, seed=1)
x = torch.from_numpy(xh).to(dev)
y = torch.full((A.m,), float("nan"), dtype=torch.float64, device=dev)
M = sp.CSRMatrix(rp, ci, va, A.n, kernel="xt")
print(M.info(), flush=True)
M.spmv(x, y)
torch.cuda.synchronize()
yr, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, xh)
bad = ~(np.abs(y.cpu().numpy() - yr) <= 1e-12 * bound)
print(w, "bad rows", int(bad.sum()), "first", np.nonzero(bad)[0][:10], flush=True)
