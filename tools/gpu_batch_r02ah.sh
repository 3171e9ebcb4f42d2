# ncu: the fused XPLAN SpMV vs the plain DOT SpMV inside cg_solve (class C)
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ah; mkdir -p $O
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 6 -c 3 -o $O/fused python tools/one_cg.py C fused 4 > $O/ncu.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $O/launches.csv python tools/one_cg.py C fused 4 > /dev/null 2>&1
