# small rank blocks: whole-range L2 prefetch on/off x persisting-L2 window over the plan
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02u; mkdir -p $O
SPMV_DEBUG=1 timeout 300 python tools/one.py S xplan 2>&1 | grep -i "persisting" | head -2 > $O/l2_attrs.txt
for cfg in "SPMV_XPLAN_L2PF=1 SPMV_XPLAN_PLANWIN=0" "SPMV_XPLAN_L2PF=0 SPMV_XPLAN_PLANWIN=0" "SPMV_XPLAN_L2PF=1 SPMV_XPLAN_PLANWIN=1" "SPMV_XPLAN_L2PF=0 SPMV_XPLAN_PLANWIN=1"; do
  for v in cgcg persist; do
    echo "$cfg $v" >> $O/proxy.jsonl
    env $cfg timeout 600 python tools/proxy_ranks.py --variant $v --ps 4,8 --ranks first >> $O/proxy.jsonl 2>> $O/proxy.err
  done
done
