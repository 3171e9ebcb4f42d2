#!/bin/bash
# XPLAN side split sweep (SPMV_XPLAN_SIDE per mille of nnz on the idle SMs): time + parity
for pm in 0 30 50 70 90 120; do
  timeout 120 python tools/time_one.py side$pm C xplan SPMV_XPLAN_SIDE=$pm 2>/dev/null | tail -1
done
for pm in 0 50 90; do
  timeout 120 python tools/time_one.py side$pm B xplan SPMV_XPLAN_SIDE=$pm 2>/dev/null | tail -1
done
SPMV_XPLAN_SIDE=70 timeout 300 python -c "
import sys; sys.path.insert(0,'.')
import torch, numpy as np, gen, oracle, paper_conf_asplos_ginsbachrsbdo18_b200 as sp
for cls in ('C','B','S'):
    A=gen.makea(cls); d=torch.device('cuda:0')
    M=sp.CSRMatrix(*(torch.from_numpy(a).to(d) for a in (A.rowptr,A.colidx,A.vals)), A.n)
    xh=gen.uniform(A.n,seed=1); x=torch.from_numpy(xh).to(d); y=torch.empty(A.m,dtype=torch.float64,device=d); M.spmv(x,y)
    r,b=oracle.spmv(A.rowptr,A.colidx,A.vals,xh); print(cls, M.info()['kernel_name'], M.info()['grid'], 'parity', bool(np.all(np.abs(y.cpu().numpy()-r)<=1e-12*b)))
"
