#!/usr/bin/env python3
"""Run a few CG solves of one variant on a NAS class (for ncu captures).
usage: one_cg.py CLASS VARIANT [ITERS]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

cls, variant = sys.argv[1], sys.argv[2]
iters = int(sys.argv[3]) if len(sys.argv) > 3 else 4
dev = torch.device("cuda:0")
A = gen.makea(cls)
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
M = sp.CSRMatrix(rp, ci, va, A.n, cg_variant=variant)
b = torch.ones(A.n, dtype=torch.float64, device=dev)
x = torch.empty_like(b)
for _ in range(3):
    M.cg_solve(b, x, max_iter=iters)
torch.cuda.synchronize()
