#!/usr/bin/env python3
"""Kernel-selection sweep (the paper's "try every API, keep the fastest",
P:275-280): times every SpMV kernel variant alone on the BASELINE configs
(CUDA events, L2 flushed before each launch) and prints one JSON line per
variant with GB/s against the algorithmic bytes.  GPU only."""
import json
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np
import torch

import gen
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

VARIANTS = [("auto", {}, {}), ("auto_noplan", {"plan": False}, {})] + \
    [(f"xplan_B{b}", {"kernel": "xplan"}, {"SPMV_XPLAN_B": str(b)}) for b in (4, 8)] + \
    [("xplan_dyn", {"kernel": "xplan"}, {"SPMV_XPLAN_DYN": "1"})] + \
    [("xt", {"kernel": "xt"}, {}), ("xt_B4", {"kernel": "xt"}, {"SPMV_XT_B": "4"})] + \
    [("sell", {"kernel": "sell"}, {}), ("sellsort", {"kernel": "sellsort"}, {}), ("merge", {"kernel": "merge"}, {})] + \
    [(f"vector{g}", {"kernel": "vector", "vec_lanes": g, "plan": False}, {}) for g in (8, 16, 32)] + \
    [(f"vector32_u{u}", {"kernel": "vector", "vec_lanes": 32, "plan": False}, {"SPMV_UNROLL": str(u)}) for u in (2, 8)] + \
    [(f"xstat_B8_G{g}_U8", {"kernel": "xstat", "plan": False}, {"SPMV_XSTAT_B": "8", "SPMV_XSTAT_G": str(g),
                                                                  "SPMV_XSTAT_U": "8"}) for g in (8,)]


def time_variant(A, x, y, kw, env, reps=20):
    for k, v in env.items():
        os.environ[k] = v
    try:
        M = sp.CSRMatrix(*A, **kw)
    finally:
        for k in env:
            os.environ.pop(k, None)
    info = M.info()
    flush = torch.empty(256 << 20, dtype=torch.int8, device="cuda")
    for _ in range(3):
        M.spmv(x, y)
    ts = []
    for _ in range(reps):
        flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        M.spmv(x, y)
        b.record()
        b.synchronize()
        ts.append(a.elapsed_time(b))
    # back to back (steady state; inputs larger than L2 stream from HBM every launch)
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps):
        M.spmv(x, y)
    b.record()
    b.synchronize()
    info["us_steady"] = a.elapsed_time(b) / reps * 1e3
    M.destroy()
    return statistics.median(ts), info


def main():
    which = sys.argv[1:] or ["B", "C", "parboil"]
    dev = torch.device("cuda:0")
    for w in which:
        if w == "parboil":
            C = gen.powerlaw()
        elif w.startswith("stencil"):
            C = gen.stencil27(int(w[7:]))
        else:
            C = gen.makea(w)
        rp = torch.from_numpy(C.rowptr).to(dev)
        ci = torch.from_numpy(C.colidx).to(dev)
        va = torch.from_numpy(C.vals).to(dev)
        x = torch.from_numpy(gen.uniform(C.n, seed=1, f32=C.vals.dtype == np.float32)).to(dev)
        y = torch.empty(C.m, dtype=va.dtype, device=dev)
        nbytes = C.bytes_per_spmv()
        if w.startswith("stencil"):
            # the matrix-free operator of the same matrix (NEXT-3): algorithmic bytes of the CSR
            # form reported for comparison, and its own 2*8 B per point
            N = int(w[7:])
            flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
            for _ in range(3):
                sp.stencil27_apply(N, N, N, x, y)
            ts = []
            for _ in range(20):
                flush.zero_()
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record()
                sp.stencil27_apply(N, N, N, x, y)
                b.record()
                b.synchronize()
                ts.append(a.elapsed_time(b))
            ms = statistics.median(ts)
            print(json.dumps({"matrix": w, "variant": "matrix_free", "kernel": "stencil27", "us": round(ms * 1e3, 2),
                              "gbs": round(nbytes / (ms / 1e3) / 1e9, 1),
                              "own_gbs": round(16 * C.m / (ms / 1e3) / 1e9, 1),
                              "gflops": round(2 * C.nnz / (ms / 1e3) / 1e9, 1)}), flush=True)
        for name, kw, env in VARIANTS:
            try:
                ms, info = time_variant((rp, ci, va, C.n), x, y, kw, env)
            except Exception as e:  # noqa
                print(json.dumps({"matrix": w, "variant": name, "error": str(e)[:200]}), flush=True)
                continue
            print(json.dumps({"matrix": w, "variant": name, "kernel": info["kernel_name"],
                              "lanes": info["vec_lanes"], "us": round(ms * 1e3, 2),
                              "us_steady": round(info["us_steady"], 2),
                              "gbs": round(nbytes / (ms / 1e3) / 1e9, 1),
                              "gflops": round(2 * C.nnz / (ms / 1e3) / 1e9, 1)}), flush=True)


if __name__ == "__main__":
    main()
