# round-2 (second session) regression: GPU suite, smoke, bench x2, launch list, ncu captures, idiom rows
cd $GRAFT_REPO_ROOT
O=gpurun_out/${OUT:-r02z3}; mkdir -p $O
timeout 3000 python -m pytest tests -m gpu -q > $O/pytest_gpu.log 2>&1; echo "rc=$?" >> $O/pytest_gpu.log
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1; echo "rc=$?" >> $O/smoke.log
timeout 900 python bench.py --steps 20 --warmup 5 > $O/bench1.json 2> $O/bench1.err
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench2.json 2> $O/bench2.err
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $O/bench_ref.json 2> $O/bench_ref.err
timeout 1500 python tools/sweep.py C B parboil > $O/sweep.jsonl 2> $O/sweep.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 30 -c 1 -o $O/xplan_cg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_cgcg -s 30 -c 1 -o $O/cgcg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
