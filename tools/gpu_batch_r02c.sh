cd $GRAFT_REPO_ROOT
O=gpurun_out/r02c; mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T odd_C C xplan
T even_C C xplan SPMV_LIB_PATH=tools/variants/lib_even.so
T odd_B B xplan
T even_B B xplan SPMV_LIB_PATH=tools/variants/lib_even.so
T odd_C2 C xplan
T even_C2 C xplan SPMV_LIB_PATH=tools/variants/lib_even.so
timeout 1500 python -m pytest tests/test_gpu_persist.py -x -q > $O/pytest_persist.log 2>&1
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant persist --ranks first > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
