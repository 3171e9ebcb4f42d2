cd $GRAFT_REPO_ROOT
O=gpurun_out/r02p; mkdir -p $O
for P in 1 8; do timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1; done
timeout 900 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
