cd $GRAFT_REPO_ROOT
O=gpurun_out/r02g; mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T B_pf0 B xplan SPMV_XPLAN_L2PF=0
T B_pf1 B xplan SPMV_XPLAN_L2PF=1
T C_pf0 C xplan SPMV_XPLAN_L2PF=0
T A_pf0 A xplan SPMV_XPLAN_L2PF=0
T A_pf1 A xplan SPMV_XPLAN_L2PF=1
for pf in 0 1; do
  SPMV_XPLAN_L2PF=$pf timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant cgcg --ranks first > $O/proxy_cgcg_pf$pf.jsonl 2> $O/proxy_pf$pf.err
done
SPMV_XPLAN_L2PF=1 timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant persist --ranks first > $O/proxy_persist_pf1.jsonl 2>> $O/proxy_pf1.err
timeout 600 python -m pytest tests/test_gpu_spmv.py -q -x -k "xplan" > $O/pytest.log 2>&1
