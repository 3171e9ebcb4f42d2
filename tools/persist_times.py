#!/usr/bin/env python3
"""Per-CTA phase timeline of one iteration of the persistent CG kernel
(k_cg_persist) on rank r's share of a P-way class run (proxy
transport): x ready, streaming done, SpMV done, grid barrier 1, update done,
grid barrier 2 -- needs a -DSPMV_TUNING variant build (SPMV_PERSIST_TIMES).
usage: persist_times.py CLASS P RANK [iters]"""
import os
import subprocess
import sys

if os.environ.get("_PT_CHILD") != "1":
    env = dict(os.environ, _PT_CHILD="1", SPMV_PERSIST_TIMES="1",
               SPMV_LIB_PATH=os.environ.get("SPMV_LIB_PATH", "tools/variants/lib_tuning.so"))
    r = subprocess.run([sys.executable, *sys.argv], env=env, capture_output=True, text=True)
    blk = r.stderr.split("[persist times]")
    print(f"{sys.argv[1:]}" + ("[persist times]" + blk[-1] if len(blk) > 1 else r.stderr[-2000:]), flush=True)
    sys.exit(r.returncode)

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

cls, P, rank = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
iters = int(sys.argv[4]) if len(sys.argv) > 4 else 25
dev = torch.device("cuda:0")
A = gen.makea(cls)
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
d = sp.Dist(rank, P, 0, transport="proxy") if P > 1 else None
M = sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel="xplan")
M.set_cg_variant("persist")
info = M.info()
nl = info["row_end"] - info["row_begin"]
b = torch.ones(nl, dtype=torch.float64, device=dev)
x = torch.empty(nl, dtype=torch.float64, device=dev)
for _ in range(3):
    M.cg_solve(b, x, iters)
torch.cuda.synchronize()
