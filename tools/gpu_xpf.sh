#!/bin/bash
# XPLAN prologue variants: L2 prefetch of the first chunks (XP_XPF) / x wait behind the first batch (XP_XDEFER)
O=gpurun_out/xpf; mkdir -p $O; : > $O/gap.txt
for rep in 1 2; do
for v in base xdefer xpf1 xpf2 xpf1defer; do
  if [ $v = base ]; then L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so; else L=tools/variants/lib_$v.so; fi
  for c in C B; do echo -n "$v " >> $O/gap.txt; SPMV_LIB_PATH=$L timeout 120 python tools/gap.py $c rand >> $O/gap.txt 2>&1; done
done; done
for v in xdefer xpf1 xpf2 xpf1defer; do
SPMV_LIB_PATH=tools/variants/lib_$v.so timeout 300 python -c "
import sys; sys.path.insert(0,'.')
import torch, numpy as np, gen, oracle, paper_conf_asplos_ginsbachrsbdo18_b200 as sp
d=torch.device('cuda:0')
for cls in ('C','B','W','S'):
    A=gen.makea(cls)
    M=sp.CSRMatrix(*(torch.from_numpy(a).to(d) for a in (A.rowptr,A.colidx,A.vals)), A.n, kernel='xplan')
    xh=gen.uniform(A.n,seed=1); x=torch.from_numpy(xh).to(d); y=torch.empty(A.m,dtype=torch.float64,device=d)
    for _ in range(3): M.spmv(x,y)
    r,b=oracle.spmv(A.rowptr,A.colidx,A.vals,xh); print('$v', cls, 'parity', bool(np.all(np.abs(y.cpu().numpy()-r)<=1e-12*b)))
" >> $O/parity.txt 2>&1
done
cat $O/gap.txt $O/parity.txt
