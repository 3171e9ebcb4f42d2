# a partial persisting window over the class-C plan (the first 128 MB, 79 MB of it persisting)
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02aq; mkdir -p $O
for W in 0 1 0 1; do
  SPMV_XPLAN_PLANWIN=$W timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/b.json 2> $O/b.err
  python -c "
import json; d=json.load(open('$O/b.json')); print('planwin=$W', d['value'], d['spmv']['us_avg'], d['e2e']['value'], d['cg_variants'])" >> $O/ab.txt
done
for W in 0 1; do echo "planwin=$W" >> $O/gap.txt; SPMV_XPLAN_PLANWIN=$W timeout 300 python tools/gap.py C rand >> $O/gap.txt 2>&1; SPMV_XPLAN_PLANWIN=$W timeout 300 python tools/gap.py B rand >> $O/gap.txt 2>&1; done
SPMV_XPLAN_PLANWIN=1 timeout 900 python tools/proxy_ranks.py --variant cgcg --ps 2 --ranks first > $O/proxy2.jsonl 2> $O/proxy2.err
