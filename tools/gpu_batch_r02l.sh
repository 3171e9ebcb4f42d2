# round 2 (re-entry): guard-region test, persistent-CG phase timelines at P = 1/2/4/8, XPLAN steady-state timelines, ncu of the P=8 persistent kernel
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02l; mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_bounds.py tests/test_gpu_sanitizer.py -q -x > $O/pytest_bounds.log 2>&1; echo "rc=$?" >> $O/pytest_bounds.log
for P in 1 2 4 8; do timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1; done
for P in 1 8; do XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C $P 0 >> $O/xplan_times_noflush.txt 2>&1; done
_PT_CHILD=1 timeout 600 ncu --set full --clock-control none -k regex:k_cg_persist -c 1 -o $O/persist_P8 python tools/persist_times.py C 8 0 > $O/ncu_persist.log 2>&1
