#!/bin/bash
# time XPLAN build variants (tools/variants/lib_*.so) on NAS class C and B; print grid/cluster
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  for mat in C B; do
    for e in "" "SPMV_XPLAN_B=8" "SPMV_XPLAN_B=6"; do
      timeout 120 python tools/time_one.py $(basename $v .so)${e:+:$e} $mat xplan $e 2>/dev/null | tail -1
    done
  done
  timeout 120 python -c "
import sys; sys.path.insert(0,'.')
import torch, gen, paper_conf_asplos_ginsbachrsbdo18_b200 as sp
A=gen.makea('C'); d=torch.device('cuda:0')
M=sp.CSRMatrix(*(torch.from_numpy(a).to(d) for a in (A.rowptr,A.colidx,A.vals)), A.n)
i=M.info(); print('$v', i['kernel_name'], i['grid'], i['cluster'])
x=torch.from_numpy(gen.uniform(A.n,seed=1)).to(d); y=torch.empty(A.m,dtype=torch.float64,device=d); M.spmv(x,y)
import oracle, numpy as np
r,b=oracle.spmv(A.rowptr,A.colidx,A.vals,gen.uniform(A.n,seed=1)); print('parity', bool(np.all(np.abs(y.cpu().numpy()-r)<=1e-12*b)))
"
done
cp /tmp/orig_lib.so $L
