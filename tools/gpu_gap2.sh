#!/bin/bash
O=gpurun_out/gap2; mkdir -p $O; : > $O/res.txt
for r in 1 2; do
timeout 200 python tools/gap2.py >> $O/res.txt 2>&1
timeout 200 python tools/gap2.py --cg >> $O/res.txt 2>&1
timeout 200 python tools/gap2.py --smi >> $O/res.txt 2>&1
timeout 200 python tools/gap2.py --cg --smi >> $O/res.txt 2>&1
timeout 200 python tools/gap2.py --reps 30 >> $O/res.txt 2>&1
done
cat $O/res.txt
