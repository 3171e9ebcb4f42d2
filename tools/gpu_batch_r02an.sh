# p2p: one publication for the r.r partials and the x slice in k_cgcg
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02an; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py tests/test_gpu_cgcg.py tests/test_gpu_cg.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_single.json 2> $O/bench_single.err
for T in p2p nccl; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$T timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29562 bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_dist1_$T.json 2> $O/bench_dist1_$T.err
done
for f in bench_single bench_dist1_p2p bench_dist1_nccl; do python -c "
import json; d=json.load(open('$O/$f.json')); print('$f', d['value'], d.get('transport'))" >> $O/ab.txt; done
timeout 900 python tools/proxy_ranks.py --variant cgcg --ps 2,8 --ranks first > $O/proxy.jsonl 2> $O/proxy.err
