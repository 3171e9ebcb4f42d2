# round-2 final: GPU suite, smoke, bench (x2), sweep, launch list, ncu captures
cd $GRAFT_REPO_ROOT
O=gpurun_out/final; mkdir -p $O
timeout 3000 python -m pytest tests -m gpu -q > $O/pytest_gpu.log 2>&1
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1
timeout 900 python bench.py --steps 20 --warmup 5 > $O/bench1.json 2> $O/bench1.err
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench2.json 2> $O/bench2.err
timeout 1500 python tools/sweep.py C B parboil > $O/sweep.jsonl 2> $O/sweep.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 30 -c 1 -o $O/xplan_cg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 2 -c 1 -o $O/xplan_alone python tools/one.py C xplan > /dev/null 2>&1
