cd $GRAFT_REPO_ROOT
O=gpurun_out/r02j; mkdir -p $O
T() { timeout 150 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T parboil_il2 parboil sellsort
T parboil_il1 parboil sellsort SPMV_LIB_PATH=tools/variants/lib_il1.so
T parboil_il2_steady parboil sellsort TIME_STEADY=1
T parboil_il1_steady parboil sellsort TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_il1.so
T st256_il2 stencil256 sell
T st256_il1 stencil256 sell SPMV_LIB_PATH=tools/variants/lib_il1.so
T B_steady_rule B xplan TIME_STEADY=1
T C_steady_rule C xplan TIME_STEADY=1
T A_steady_rule A xplan TIME_STEADY=1
timeout 1500 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_cg.py -q -x > $O/pytest.log 2>&1
timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant persist --ranks first > $O/proxy_persist.jsonl 2> $O/proxy.err
