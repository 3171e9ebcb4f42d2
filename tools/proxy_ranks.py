#!/usr/bin/env python3
"""Per-rank proxy of the row-sharded NAS CG class-C run on ONE GPU
(VERDICT r1 "Next" 1c).

For P in {1, 2, 4, 8} and a rank r, a handle created with the proxy transport
(spmv_dist_init_proxy) does exactly rank r's share of the P-way run -- its
nnz-balanced row block, the padded x layout of P*maxlen columns, the same
plan, kernels and launch shapes -- with every exchange skipped.  Timed with
CUDA events on the launching stream:
  spmv_us    one SpMV of the rank's block (L2 flushed before; includes the
             copy of the x slice into the padded buffer, ~m/P*8 bytes)
  spmv_graph_us  the same call 20 times back to back from a CUDA graph (steady
             state, as inside CG: a block of <= 96 MB stays L2-resident)
  cg_it_us   one CG iteration inside the NPB step (K steps of 25 iterations
             + residual SpMV, back to back, divided by 25*K)
and the implied upper bound on strong-scaling efficiency from compute alone,
  eff_compute = T_1 / (P * T_P)  (T = cg_it_us; communication excluded).
usage: proxy_ranks.py [--kernel auto|xplan|xt] [--steps K] [--cls C] > jsonl
"""
import argparse
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import gen  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402


def _peak():
    try:
        return float(json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                                 "MEASURED_PEAKS.json")))["hbm_gbs"])
    except (OSError, KeyError, ValueError):
        return 6534.1


PEAK = _peak()


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--kernel", default="auto")
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--cls", default="C")
    ap.add_argument("--ranks", default="first,last")
    ap.add_argument("--variant", default="cgcg")
    ap.add_argument("--ps", default="1,2,4,8", help="rank counts P to run")
    args = ap.parse_args()
    dev = torch.device("cuda:0")
    na, nonzer, niter, shift = gen.NPB_CLASSES[args.cls]
    A = gen.makea(args.cls)
    rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
    flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
    stream = torch.cuda.Stream(dev)  # non-default: the graph-timed leg captures on it
    torch.cuda.set_stream(stream)  # every handle launches on the stream current at its creation
    t1 = None
    for P in [int(v) for v in args.ps.split(",")]:
        ranks = sorted({0 if s == "first" else P - 1 for s in args.ranks.split(",")})
        for r in ranks:
            d = sp.Dist(r, P, 0, transport="proxy")
            M = sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel=args.kernel)
            M.set_cg_variant(args.variant)
            info = M.info()
            nl = info["row_end"] - info["row_begin"]
            x = torch.from_numpy(gen.uniform(A.n, seed=5)[info["row_begin"]:info["row_end"]].copy()).to(dev)
            y = torch.empty(nl, dtype=torch.float64, device=dev)
            for _ in range(3):
                M.spmv(x, y)
            ts = []
            for _ in range(20):
                flush.zero_()
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record(stream)
                M.spmv(x, y)
                b.record(stream)
                b.synchronize()
                ts.append(a.elapsed_time(b))
            spmv_us = statistics.median(ts) * 1e3
            # steady state, as inside the CG loop and as bench.py's us_avg: 20 back-to-back
            # calls (each = slice copy into the padded x + the SpMV) replayed from a CUDA graph
            g = torch.cuda.CUDAGraph()
            with torch.cuda.graph(g, stream=stream):
                for _ in range(20):
                    M.spmv(x, y)
            g.replay()
            tg = []
            for _ in range(5):
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record(stream)
                g.replay()
                b.record(stream)
                b.synchronize()
                tg.append(a.elapsed_time(b) * 1e3 / 20)
            spmv_graph_us = statistics.median(tg)
            del g
            xv = torch.ones(nl, dtype=torch.float64, device=dev)
            z = torch.empty_like(xv)
            out2 = torch.zeros(2, dtype=torch.float64, device=dev)
            for _ in range(3):
                M.npb_outer(xv, z, 25, shift, out2)
            xv.fill_(1.0)
            torch.cuda.synchronize()
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record(stream)
            for _ in range(args.steps):
                M.npb_outer(xv, z, 25, shift, out2)
            b.record(stream)
            b.synchronize()
            step_ms = a.elapsed_time(b) / args.steps
            cg_it_us = step_ms * 1e3 / 25.0
            if P == 1:
                t1 = cg_it_us
            bytes_loc = info["nnz_local"] * 12 + 4 * (nl + 1) + 8 * A.n + 8 * nl
            rec = {"cls": args.cls, "P": P, "rank": r, "kernel": info["kernel_name"], "cluster": info["cluster"],
                   "m_local": nl, "nnz_local": info["nnz_local"], "spmv_us": round(spmv_us, 2),
                   "spmv_frac_copy_peak": round(bytes_loc / (spmv_us * 1e-6) / 1e9 / PEAK, 3),
                   "spmv_graph_us": round(spmv_graph_us, 2),
                   "spmv_graph_frac_copy_peak": round(bytes_loc / (spmv_graph_us * 1e-6) / 1e9 / PEAK, 3),
                   "step_ms": round(step_ms, 4), "cg_it_us": round(cg_it_us, 2),
                   "cg_its_per_s_job": round(P * 1e6 / cg_it_us, 1),
                   "eff_compute": round(t1 / (P * cg_it_us), 3) if t1 else None}
            print(json.dumps(rec), flush=True)
            M.destroy()
            d.close()


if __name__ == "__main__":
    main()
