#!/usr/bin/env python3
"""Device timing of the NEXT-4 idiom kernels (include/idioms.h) on the paper's
workloads, one JSON line per workload:

  ep_C        NAS EP class C, 2^32 Gaussian pairs (ep_npb)              pairs/s   alu
  is_C        NAS IS class C key counting, 2^27 keys into 2^23 bins      keys/s    hbm
  histo       Parboil-histo-shaped image, 996x1040 keys, 4096x256 uint8 saturating bins
  dot_2p27    scalar reduction: fp64 dot of two 2^27 vectors (2 GiB)    GB/s      hbm

CUDA events on the launching stream around each call, median of REPS after 3
warm-ups; L2 flushed (256 MiB write) before every timed call, outside the
events.  Roofline `achieved` = ALGORITHMIC bytes / time (hbm) against
MEASURED_PEAKS.json hbm_gbs.  The oracle (test infrastructure) is timed on a
bounded sample on the host for `cpu_baseline`.  Not the driver's bench.py
(which times the CG hot path); results go to profiles/ by hand.
usage: bench_idioms.py [--reps N] [--no-cpu] [workload ...]
"""
import argparse
import json
import os
import statistics
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np
import torch

import gen
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp


def peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            return json.load(f)
    except OSError:
        return {"hbm_gbs": 7672.0}


def timed(fn, reps, flush):
    for _ in range(3):
        fn()
    s = torch.cuda.current_stream()
    ts = []
    for _ in range(reps):
        flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(s)
        fn()
        b.record(s)
        b.synchronize()
        ts.append(a.elapsed_time(b) * 1e3)
    return statistics.median(ts), min(ts)


def line(name, us, us_min, units, unit_name, bytes_alg, extra, cpu=None):
    pk = peaks()
    d = {"workload": name, "us_median": round(us, 2), "us_min": round(us_min, 2),
         "value": round(units / (us * 1e-6), 1), "unit": unit_name}
    if bytes_alg:
        gbs = bytes_alg / (us * 1e-6) / 1e9
        d["roofline"] = {"bound": "hbm", "achieved": round(gbs, 1), "peak": pk["hbm_gbs"], "unit": "GB/s",
                         "frac": round(gbs / pk["hbm_gbs"], 4), "bytes_per_launch": int(bytes_alg)}
    d.update(extra)
    if cpu:
        d["cpu_baseline"] = cpu
    print(json.dumps(d), flush=True)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--reps", type=int, default=20)
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("which", nargs="*", default=["ep_C", "is_C", "histo", "dot_2p27", "jds_parboil", "stencil256",
                                                 "spmv_B", "spmv_parboil", "spmv_stencil256"])
    args = ap.parse_args()
    dev = torch.device("cuda:0")
    torch.cuda.set_device(dev)
    flush = torch.empty(256 << 20, dtype=torch.int8, device=dev)
    cpu_ok = not args.no_cpu
    if cpu_ok:
        import oracle

    if "ep_C" in args.which:
        M = gen.NPB_EP_CLASSES["C"]
        out = torch.empty(12, dtype=torch.float64, device=dev)
        ws = torch.zeros(sp.ep_npb_workspace(), dtype=torch.uint8, device=dev)
        us, us_min = timed(lambda: sp.ep_npb(M, out=out, workspace=ws), max(5, args.reps // 2), flush)
        r = out.cpu().numpy()
        cpu = None
        if cpu_ok:
            t = time.perf_counter()
            oracle.ep(24)
            dt = time.perf_counter() - t
            cpu = {"value": round((1 << 24) / dt, 1), "unit": "pairs/s", "cores": 1, "kind": "oracle",
                   "sample": f"NAS EP class S (2^24 pairs) in {dt:.2f} s, oracle/oracle_idioms.c -O3 1 thread"}
        line("NAS EP class C (2^32 pairs)", us, us_min, float(1 << M), "pairs/s", 0,
             {"sx": r[10], "sy": r[11], "gaussian_pairs": float(r[:10].sum()), "bound": "alu"}, cpu)

    if "is_C" in args.which:
        lk, lm = gen.NPB_IS_CLASSES["C"]
        keys = torch.from_numpy(gen.is_keys("C")).to(dev)
        bins = torch.zeros(1 << lm, dtype=torch.uint32, device=dev)
        us, us_min = timed(lambda: sp.idl_histogram("count", keys, bins), args.reps, flush)
        cpu = None
        if cpu_ok:
            k = keys.cpu().numpy()
            t = time.perf_counter()
            oracle.hist_count_u32(k, 1 << lm)
            dt = time.perf_counter() - t
            cpu = {"value": round(k.size / dt, 1), "unit": "keys/s", "cores": 1, "kind": "oracle",
                   "sample": f"the same 2^27 keys in {dt:.2f} s, 1 thread"}
        line("NAS IS class C key counting (2^27 keys, 2^23 uint32 bins)", us, us_min, float(1 << lk), "keys/s",
             4 * (1 << lk) + 8 * (1 << lm), {}, cpu)

    if "histo" in args.which:
        img = torch.from_numpy(gen.histo_image()).to(dev)
        nb = gen.HISTO_NBINS
        bins = torch.zeros(nb, dtype=torch.uint8, device=dev)
        ws = torch.zeros(sp.idl_histogram_workspace("sat_u8", img.numel(), nb), dtype=torch.uint8, device=dev)
        us, us_min = timed(lambda: sp.idl_histogram("sat_u8", img, bins, workspace=ws), args.reps, flush)
        cpu = None
        if cpu_ok:
            k = img.cpu().numpy()
            t = time.perf_counter()
            for _ in range(20):
                oracle.hist_sat_u8(k, nb)
            dt = (time.perf_counter() - t) / 20
            cpu = {"value": round(k.size / dt, 1), "unit": "keys/s", "cores": 1, "kind": "oracle",
                   "sample": f"the same image, 20 runs, {dt * 1e3:.2f} ms each, 1 thread"}
        line("Parboil-histo-shaped saturating histogram (996x1040 keys, 4096x256 uint8 bins)", us, us_min,
             float(img.numel()), "keys/s", 4 * img.numel() + 2 * nb, {"launches": 2}, cpu)

    if "dot_2p27" in args.which:
        n = 1 << 27
        a = torch.rand(n, dtype=torch.float64, device=dev)
        b = torch.rand(n, dtype=torch.float64, device=dev)
        out = torch.empty(1, dtype=torch.float64, device=dev)
        ws = torch.zeros(sp.idl_reduce_workspace(n), dtype=torch.uint8, device=dev)
        us, us_min = timed(lambda: sp.idl_reduce(a, b, out=out, workspace=ws), args.reps, flush)
        cpu = None
        if cpu_ok:
            ah, bh = a[: n // 8].cpu().numpy(), b[: n // 8].cpu().numpy()
            t = time.perf_counter()
            oracle.reduce(ah, bh)
            dt = time.perf_counter() - t
            cpu = {"value": round(16 * ah.size / dt / 1e9, 2), "unit": "GB/s", "cores": 1, "kind": "oracle",
                   "sample": f"2^24-element dot in {dt * 1e3:.1f} ms, 1 thread"}
        line("scalar reduction: fp64 dot, 2^27 elements", us, us_min, 16.0 * n / 1e9, "GB/s", 16 * n, {}, cpu)

    if "jds_parboil" in args.which:
        A = gen.powerlaw()
        J = gen.csr_to_jds(A)
        dv = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)
        M = sp.JDSMatrix(dv(J.perm), dv(J.jds_ptr), dv(J.zcnt), dv(J.indices), dv(J.data), J.m, J.n)
        x = dv(gen.uniform(A.n, seed=5, f32=True))
        y = torch.empty(A.m, dtype=torch.float32, device=dev)
        us, us_min = timed(lambda: M.spmv(x, y), args.reps, flush)
        # the method's algorithmic bytes of the CSR SpMV: nnz*8 + 4(m+1) + 4n + 4m
        alg = A.nnz * 8 + 4 * (A.m + 1) + 4 * A.n + 4 * A.m
        line("Parboil-shaped SpMV on the JDS-32 layout (fp32, 2^20 rows, 11.5M nnz)", us, us_min, 2.0 * A.nnz / 1e9,
             "GFLOP/s", alg, {"jds_entries": int(J.jds_ptr[-1]), "depth": J.depth})
        M.destroy()

    if "stencil256" in args.which:
        N = 256
        x = torch.rand(N ** 3, dtype=torch.float64, device=dev)
        y = torch.empty_like(x)
        us, us_min = timed(lambda: sp.stencil27_apply(N, N, N, x, y), args.reps, flush)
        # the matrix-free operator's own bytes: x once + y once (16 B per point, fp64)
        line("matrix-free 27-point stencil 256^3 fp64 (R19 weights)", us, us_min, float(N ** 3), "points/s",
             16 * N ** 3, {}, None)

    for w in ("B", "parboil", "stencil256"):
        if f"spmv_{w}" not in args.which:
            continue
        A = gen.powerlaw() if w == "parboil" else gen.stencil27(256) if w == "stencil256" else gen.makea(w)
        dv = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)
        M = sp.CSRMatrix(dv(A.rowptr), dv(A.colidx), dv(A.vals), A.n)
        x = dv(gen.uniform(A.n, seed=1, f32=A.vals.dtype == np.float32))
        y = torch.empty(A.m, dtype=x.dtype, device=dev)
        us, us_min = timed(lambda: M.spmv(x, y), args.reps, flush)
        line(f"CSR SpMV {w} ({M.info()['kernel_name']}, {'fp32' if A.vals.dtype == np.float32 else 'fp64'})", us,
             us_min, 2.0 * A.nnz / 1e9, "GFLOP/s", A.bytes_per_spmv(), {"nnz": int(A.nnz)}, None)
        M.destroy()
        del A


if __name__ == "__main__":
    main()
