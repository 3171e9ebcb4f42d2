#!/usr/bin/env python3
"""Per-CTA timeline of one XPLAN SpMV (globaltimer stamps: start, x ready,
streaming done, end) summarised over CTAs -- needs a -DSPMV_TUNING variant
build (SPMV_XPLAN_TIMES).  usage: xplan_times.py CLASS P RANK"""
import os
import re
import subprocess
import sys

if os.environ.get("_XT_CHILD") != "1":
    env = dict(os.environ, _XT_CHILD="1", SPMV_XPLAN_TIMES="1",
               SPMV_LIB_PATH=os.environ.get("SPMV_LIB_PATH", "tools/variants/lib_tuning.so"))
    r = subprocess.run([sys.executable, *sys.argv], env=env, capture_output=True, text=True)
    blocks = r.stderr.split("[xplan times]")
    if os.environ.get("XT_PER_CLUSTER") == "1":  # per-cluster end of streaming (max over its CTAs), every launch
        for blk in blocks[1:]:
            cl = {}
            for l in blk.splitlines():
                f = l.split()
                if f and f[0] == "cta":
                    cl.setdefault(int(f[3]), []).append(float(f[6]))
            print("per-cluster streamed max:", " ".join(f"{max(v):.1f}" for _, v in sorted(cl.items())))
    last = blocks[-1]
    if os.environ.get("XT_DUMP"):  # the last launch's per-CTA lines
        with open(os.environ["XT_DUMP"], "a") as f:
            f.write(last)
    span = re.search(r"kernel span ([0-9.]+) us", last)
    rows = [list(map(float, l.split()[4:8])) for l in last.splitlines() if l.strip().startswith("cta")]
    import statistics as st
    cols = list(zip(*rows))
    print(f"{sys.argv[1:]} kernel span {span.group(1) if span else '?'} us; CTAs {len(rows)}; "
          + "; ".join(f"{nm} med {st.median(c):.2f} max {max(c):.2f}" for nm, c in
                      zip(("start", "xready", "streamed", "end"), cols)))
    sys.exit(r.returncode)

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

cls, P, rank = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
dev = torch.device("cuda:0")
A = gen.makea(cls)
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
d = sp.Dist(rank, P, 0, transport="proxy") if P > 1 else None
M = sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel="xplan")
info = M.info()
nl = info["row_end"] - info["row_begin"]
x = torch.ones(nl, dtype=torch.float64, device=dev)
y = torch.empty(nl, dtype=torch.float64, device=dev)
flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
for _ in range(int(os.environ.get("XT_REPS", "3"))):
    if os.environ.get("XT_NOFLUSH") != "1":  # XT_NOFLUSH=1: back-to-back launches (steady state)
        flush.zero_()
    M.spmv(x, y)
torch.cuda.synchronize()
