#!/bin/bash
for i in 1 2 3; do for m in C B; do echo "== $m $i"; timeout 25 python tools/one.py $m xplan > /tmp/o.txt 2>&1; echo "rc $?"; grep -i "timeout" /tmp/o.txt | head -2; done; done
