#!/bin/bash
O=gpurun_out/b3; mkdir -p $O
timeout 900 python bench.py > $O/bench.json 2> $O/bench.err
SPMV_BENCH_FORCE_DIST=1 timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_nccl.json 2> $O/bench_dist1_nccl.err
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29556 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_p2p.json 2> $O/bench_dist1_p2p.err
timeout 900 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py tests/test_gpu_persist.py -q -x > $O/pytest.log 2>&1
python - <<'PY'
import json
for f in ("bench", "bench_dist1_nccl", "bench_dist1_p2p"):
    try:
        d = json.loads(open(f"gpurun_out/b3/{f}.json").read().strip().splitlines()[-1])
        print(f, d["value"], d["spmv"]["us_avg"], d["spmv"].get("us_avg_method"), d["spmv"].get("us_eager_avg"), d["spmv"]["us_flushed_median"], d["roofline"]["frac"], d["e2e"]["value"], d.get("cg_variants"), d.get("clocks"))
    except Exception as e:
        print(f, "ERR", e)
PY
grep -i "capture failed" $O/*.err; tail -2 $O/pytest.log
