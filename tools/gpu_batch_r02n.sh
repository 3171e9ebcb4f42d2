# A/B in one run: persistent CG V1/V2, XPLAN bank spreading on/off
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02n; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_persist.py tests/test_gpu_cgcg.py tests/test_gpu_spmv.py tests/test_gpu_bounds.py -q -x -k "xplan or persist or cgcg or full or guard" > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for PERM in 0 1; do for cls in C B; do echo "perm=$PERM" >> $O/gap.txt; SPMV_XPLAN_PERM=$PERM timeout 300 python tools/gap.py $cls rand >> $O/gap.txt 2>&1; done; done
for P in 1 8; do for PERM in 0 1; do for V in 1 2; do
  echo "perm=$PERM V=$V" >> $O/persist_times.txt; SPMV_XPLAN_PERM=$PERM SPMV_PERSIST_V=$V timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1
done; done; done
SPMV_XPLAN_PERM=0 timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_perm0.json 2> $O/bench0.err
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_perm1.json 2> $O/bench1.err
