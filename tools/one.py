#!/usr/bin/env python3
"""Run one SpMV variant a few times (for ncu captures).
usage: one.py MATRIX KERNEL [ENV=VAL ...]   e.g. one.py C xstat SPMV_XSTAT_B=8"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
for kv in sys.argv[3:]:
    k, v = kv.split("=")
    os.environ[k] = v
import numpy as np
import torch

import gen
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

w, kern = sys.argv[1], sys.argv[2]
C = gen.powerlaw() if w == "parboil" else gen.stencil27(int(w[7:])) if w.startswith("stencil") else gen.makea(w)
dev = torch.device("cuda:0")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (C.rowptr, C.colidx, C.vals))
x = torch.from_numpy(gen.uniform(C.n, seed=1, f32=C.vals.dtype == np.float32)).to(dev)
y = torch.empty(C.m, dtype=va.dtype, device=dev)
lanes = 0
if kern.startswith("vector") and kern != "vector":
    lanes = int(kern[6:])
    kern = "vector"
M = sp.CSRMatrix(rp, ci, va, C.n, kernel=kern, vec_lanes=lanes)
print(M.info(), file=sys.stderr)
flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
for _ in range(5):
    flush.zero_()
    M.spmv(x, y)
torch.cuda.synchronize()
