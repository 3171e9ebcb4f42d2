#!/usr/bin/env python3
"""Benchmark: NAS CG class C (fp64) on the B200 SpMV/CG library.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]

Workload (BASELINE.json metric "CSR SpMV GB/s & % HBM peak (NAS CG class C
fp64); CG iters/s at 1/2/4/8 GPU", config BJ.cfg[3]): the NAS CG class-C
matrix (exact NPB makea, n = 150,000, 36,121,058 nnz), fp64.  One STEP is one
NAS CG outer iteration = every row of SURVEY 8(a): 25 CG iterations (SpMV +
2 dots + 3 axpys each, a2/a3), the residual SpMV and the zeta/normalisation
tail (a4), row-sharded over N GPUs (a5: NCCL by default, SPMV_TRANSPORT=p2p
for the library's peer-memory kernels); the handle is
created once (a1, device-resident A, the paper's lazy copying P:1175-1184).

value  = CG iterations per second of the whole job (25 per step; the residual
         SpMV is timed but not counted, reading R23): K steps back to back
         between two CUDA events on the launching stream (A is larger than
         L2, so no flush is needed between steps), max over ranks.
e2e    = the same metric through the public API with HOST buffers: x copied in
         from pinned memory and x, z, {zeta, rnorm} copied back every step.
roofline = the SpMV kernel (the dominant kernel, ~97% of the step's bytes),
         timed alone with CUDA events on the launching stream: back-to-back
         launches replayed from a CUDA graph, as the CG step launches them
         (A's plan is larger than L2, streamed from HBM every time) -> us_avg
         (us_eager_avg: the same launches issued eagerly), and each launch
         after a 256 MiB write flush -> us_flushed_median; algorithmic bytes /
         us_avg vs the measured HBM copy bandwidth of MEASURED_PEAKS.json.
cpu_baseline = the CPU oracle on a bounded sample: its OpenMP copy on all host cores
         (value) and the plain oracle on 1 thread (single_thread).
`--impl reference` times the oracle itself as the reference arm.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "CSR SpMV GB/s & % HBM peak (NAS CG class C fp64); CG iters/s at 1/2/4/8 GPU"
UNIT = "CG iters/s"
CLS = "C"
NOMINAL_HBM_GBS = 8000.0
FLUSH_BYTES = 256 << 20  # > 126 MB L2


def log(*a):
    print(*a, file=sys.stderr, flush=True)


class stdout_to_stderr:
    """Route fd 1 to fd 2 while NCCL initialises: NCCL may print its version
    banner on stdout, and the bench contract is one JSON line on stdout."""

    def __enter__(self):
        sys.stdout.flush()
        self.saved = os.dup(1)
        os.dup2(2, 1)
        return self

    def __exit__(self, *a):
        sys.stdout.flush()
        os.dup2(self.saved, 1)
        os.close(self.saved)


def measured_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        with open(p) as f:
            d = json.load(f)
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs, copy read+write)"
    except Exception:
        return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


def workload_config(A, n_gpus):
    na, nonzer, niter, shift = __import__("gen").NPB_CLASSES[CLS]
    return {
        "workload": f"NAS CG class {CLS} (makea NA={na}, NONZER={nonzer}, SHIFT={shift}), fp64 CG, "
                    f"1 step = 1 NPB outer iteration (25 CG its + residual SpMV)",
        "n": int(A.n), "nnz": int(A.nnz), "cgitmax": 25,
        "bytes_per_spmv": int(A.bytes_per_spmv()),
        "l2": "inputs larger than L2: A = 436 MB as CSR (382 MB as the plan) > 126 MB L2; the K steps run back "
              "to back (no flush); the roofline leg times back-to-back SpMVs the same way (us_avg) and, "
              "pessimistically, each after a 256 MiB write flush (us_flushed_median)",
        "parallelism": f"row-shard x{n_gpus} (nnz-balanced); x all-gather + dot all-reduces over peer memory "
                       f"(p2p kernels) or NCCL",
    }


# ------------------------------------------------------------------ clocks
class ClockSampler:
    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu_index: int):
        self.gpu = gpu_index
        self.proc = None
        self.lines = []

    def start(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.gpu), f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-lms", "50"], stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self):
        if not self.proc:
            return None
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except Exception:
            self.proc.kill()
        self.t.join(timeout=2)
        sm, mx, reasons = [], 0.0, set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            f = [x.strip() for x in ln.split(",")]
            if len(f) < 9:
                continue
            try:
                sm.append(float(f[1]))
                mx = max(mx, float(f[2]))
            except ValueError:
                continue
            for nm, v in zip(names, f[5:9]):
                if v.lower().startswith("active"):
                    reasons.add(nm)
        if not sm:
            return None
        return {"sm_mhz": statistics.median(sm), "sm_max_mhz": mx, "reasons": sorted(reasons),
                "samples": len(sm)}


# --------------------------------------------------------------- our arm
def run_ours(args):
    import numpy as np
    import torch
    import torch.distributed as dist

    import gen
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if world != args.gpus:
        log(f"note: --gpus {args.gpus} but WORLD_SIZE={world}; using WORLD_SIZE")
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    # one non-default stream for everything (torch ops, the handle's launches,
    # the events): the roofline leg captures SpMV launches into a CUDA graph,
    # which the legacy default stream cannot do
    torch.cuda.set_stream(torch.cuda.Stream(dev))
    d = None
    # SPMV_BENCH_FORCE_DIST=1 runs the row-sharded NCCL path even with one rank
    # (how the multi-GPU code is exercised on the 1-GPU development box)
    use_dist = world > 1 or os.environ.get("SPMV_BENCH_FORCE_DIST") == "1"
    # transport of the row-sharded exchange: "nccl" (default, measured faster
    # at one rank) or "p2p" (our kernels over CUDA-IPC peer memory / NVLink)
    # (1-rank measurement: NCCL 12.38k vs p2p 11.57k vs single 12.83k CG it/s)
    transport = os.environ.get("SPMV_TRANSPORT", "nccl")
    if use_dist:
        with stdout_to_stderr():
            dist.init_process_group("nccl", device_id=dev, rank=rank, world_size=world)
            d = sp.Dist(rank, world, local, transport=transport)
            dist.barrier(device_ids=[local])

    na, nonzer, niter, shift = gen.NPB_CLASSES[CLS]
    t0 = time.time()
    A = gen.makea(CLS)
    log(f"[rank {rank}] generated class {CLS}: n={A.n} nnz={A.nnz} in {time.time() - t0:.1f}s")
    rp = torch.from_numpy(A.rowptr).to(dev)
    ci = torch.from_numpy(A.colidx).to(dev)
    va = torch.from_numpy(A.vals).to(dev)
    try:
        M = sp.CSRMatrix(rp, ci, va, A.n, dist=d)
    except sp.SpmvError as e:
        if d is None or transport != "p2p":
            raise
        # peer mappings unavailable on this node: the NCCL transport (all ranks agree)
        log(f"[rank {rank}] p2p transport unavailable ({e}); using NCCL")
        d.close()
        transport = "nccl"
        with stdout_to_stderr():
            d = sp.Dist(rank, world, local, transport="nccl")
        M = sp.CSRMatrix(rp, ci, va, A.n, dist=d)
    M.set_cg_variant(args.cg_variant)
    info = M.info()
    b0, b1 = info["row_begin"], info["row_end"]
    nl = b1 - b0
    flush = torch.empty(FLUSH_BYTES // 4, dtype=torch.int32, device=dev)
    stream = torch.cuda.current_stream(dev)

    def barrier():
        torch.cuda.synchronize(dev)
        if use_dist:
            dist.barrier(device_ids=[local])
        torch.cuda.synchronize(dev)

    def max_over_ranks(v: float) -> float:
        if not use_dist:
            return v
        t = torch.tensor([v], dtype=torch.float64, device=dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    # ---------------- device-resident NAS CG steps (value)
    x = torch.ones(nl, dtype=torch.float64, device=dev)
    z = torch.empty(nl, dtype=torch.float64, device=dev)
    out2 = torch.zeros(2, dtype=torch.float64, device=dev)
    clocks = ClockSampler(local)
    clocks.start()
    for _ in range(args.warmup):
        M.npb_outer(x, z, 25, shift, out2)
    barrier()
    x.fill_(1.0)
    # A (436 MB as CSR, 382 MB as the plan) is larger than the 126 MB L2, so
    # the K steps run back to back in one event-bracketed region (no flush:
    # the timing rules' "inputs larger than L2" option)
    ev0, ev1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    launches0 = sp.launch_count()
    barrier()
    ev0.record(stream)
    for k in range(args.steps):
        M.npb_outer(x, z, 25, shift, out2)
    ev1.record(stream)
    barrier()
    launches = sp.launch_count() - launches0
    M.cg_status()
    t_ms = max_over_ranks(ev0.elapsed_time(ev1))
    zeta_last = float(out2[0].item())
    value = 25.0 * args.steps / (t_ms / 1e3)

    # the other CG variants (NEXT-1: single reduction, persistent), same protocol, reported beside the headline
    variants = {args.cg_variant: round(value, 2)}
    for other in [v for v in ("textbook", "cgcg", "persist") if v != args.cg_variant]:
        M.set_cg_variant(other)
        x.fill_(1.0)
        for _ in range(args.warmup):
            M.npb_outer(x, z, 25, shift, out2)
        x.fill_(1.0)
        barrier()
        ev0.record(stream)
        for k in range(args.steps):
            M.npb_outer(x, z, 25, shift, out2)
        ev1.record(stream)
        barrier()
        M.cg_status()
        t_other = max_over_ranks(ev0.elapsed_time(ev1))
        variants[other] = round(25.0 * args.steps / (t_other / 1e3), 2)
        variants[f"zeta_last_{other}"] = float(out2[0].item())
    M.set_cg_variant(args.cg_variant)

    # ---------------- e2e through the public API with host buffers
    xh = torch.ones(nl, dtype=torch.float64).pin_memory()
    zh = torch.empty(nl, dtype=torch.float64).pin_memory()
    o2h = torch.zeros(2, dtype=torch.float64).pin_memory()
    M.npb_outer(xh, zh, 25, shift, o2h)  # warm the staged path
    xh.fill_(1.0)
    barrier()
    e2e_ms = 0.0
    for k in range(args.steps):
        flush.zero_()
        barrier()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(stream)
        M.npb_outer(xh, zh, 25, shift, o2h)  # H2D x, graph, D2H x, z, out2 (synchronous)
        b.record(stream)
        b.synchronize()
        e2e_ms += a.elapsed_time(b)
    e2e_ms = max_over_ranks(e2e_ms)
    e2e_val = 25.0 * args.steps / (e2e_ms / 1e3)

    # ---------------- roofline: the SpMV kernel timed alone
    p = torch.from_numpy(gen.uniform(A.n, seed=5)[b0:b1].copy()).to(dev)
    q = torch.empty(nl, dtype=torch.float64, device=dev)
    reps = max(10, args.steps)
    for _ in range(3):
        M.spmv(p, q)
    # (1) steady state, as inside the CG step: `reps` launches back to back
    #     between two events on the launching stream.  A's plan (382 MB) is
    #     larger than the 126 MB L2 and streamed in the same order every time,
    #     so every launch reads it from HBM ("inputs larger than L2"; ncu's
    #     cold-cache DRAM bytes per launch agree, profiles/spmv_traffic.json).
    #     Launched as the CG step launches it -- from a CUDA graph (the `reps`
    #     launches captured once, replayed between the events); the eager
    #     back-to-back time is reported beside it (it adds ~2 us of launch gap
    #     per call: kernel span from globaltimer stamps 67.5 us, graph 67.9,
    #     eager 70.1 on one box)
    barrier()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record(stream)
    for _ in range(reps):
        M.spmv(p, q)
    b.record(stream)
    b.synchronize()
    sp_eager = a.elapsed_time(b) / reps
    sp_steady, us_method = sp_eager, "eager back-to-back launches"
    try:
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=stream):
            for _ in range(reps):
                M.spmv(p, q)
        g.replay()
        barrier()
        per = []
        for _ in range(5):  # median of 5 replays of `reps` launches each
            a.record(stream)
            g.replay()
            b.record(stream)
            b.synchronize()
            per.append(a.elapsed_time(b) / reps)
        sp_steady = statistics.median(per)
        us_method = f"CUDA-graph replay of {reps} back-to-back launches, median of 5 replays"
    except Exception as e:  # capture unsupported on this path: keep the eager number, say so
        log(f"[rank {rank}] roofline graph capture failed ({e}); using eager launches")
    # (2) cold, pessimistic: a 256 MiB write queued ahead of each launch (its
    #     dirty lines are written back while the kernel streams)
    sp_ms = []
    for _ in range(reps):
        barrier()
        flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(stream)
        M.spmv(p, q)
        b.record(stream)
        b.synchronize()
        sp_ms.append(a.elapsed_time(b))
    clk = clocks.stop()
    # algorithmic bytes of this rank's launch: local nnz*(8+4) + 4*(m_loc+1) + 8*n (x) + 8*m_loc (y)
    nnz_loc = info["nnz_local"]
    spmv_bytes = nnz_loc * 12 + 4 * (nl + 1) + 8 * A.n + 8 * nl
    sp_avg = max_over_ranks(sp_steady)
    sp_eager_max = max_over_ranks(sp_eager)
    sp_flushed = statistics.median(sp_ms)
    achieved = spmv_bytes / (sp_avg / 1e3) / 1e9
    peak, peak_src = measured_peaks()
    traffic = None
    tf = os.path.join(ROOT, "profiles", "spmv_traffic.json")
    if os.path.exists(tf) and world == 1:
        try:
            tj = json.load(open(tf))
            traffic = tj.get(f"class{CLS}:{info['kernel_name']}")
        except Exception:
            traffic = None

    # ---------------- CPU oracle baseline (rank 0, N=1 only)
    cpu = None
    if world == 1 and not args.no_cpu:
        cpu = cpu_baseline(A, shift, budget_s=args.cpu_budget)

    if rank == 0:
        line = {
            "metric": METRIC, "value": round(value, 2), "unit": UNIT, "n_gpus": world,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": round(t_ms / args.steps, 4),
            "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "f64",
            "data": "synthetic (exact NPB makea class C generator, seeded)",
            "config": workload_config(A, world),
            "impl": "ours",
            "distributed_path": bool(use_dist),
            "transport": transport if use_dist else None,
            "kernel": {"name": info["kernel_name"], "vec_lanes": info["vec_lanes"], "grid": info["grid"]},
            "spmv": {
                "gbs": round(achieved, 1), "gflops": round(2 * nnz_loc / (sp_avg / 1e3) / 1e9, 1),
                "us_avg": round(sp_avg * 1e3, 2),
                "us_avg_method": us_method,
                "us_eager_avg": round(sp_eager_max * 1e3, 2),
                "us_flushed_median": round(sp_flushed * 1e3, 2),
                "gbs_flushed": round(spmv_bytes / (sp_flushed / 1e3) / 1e9, 1),
                "pct_of_8TBs": round(100 * achieved / NOMINAL_HBM_GBS, 2),
                "pct_of_measured_copy": round(100 * achieved / peak, 2),
                "bytes_per_launch": int(spmv_bytes),
            },
            "cg_gbs_effective": round(value * (spmv_bytes + 10 * 8 * nl) / 1e9 * world, 1),
            "roofline": {"bound": "hbm", "achieved": round(achieved, 1), "peak": peak, "unit": "GB/s",
                         "frac": round(achieved / peak, 4), "traffic": traffic,
                         # the kernel's own DRAM rate: ncu bytes per launch (the plan is smaller than
                         # the CSR arrays) over the same launch time
                         "achieved_dram": (round(traffic / (sp_avg / 1e3) / 1e9, 1) if traffic else None),
                         "frac_dram": (round(traffic / (sp_avg / 1e3) / 1e9 / peak, 4) if traffic else None),
                         "peak_source": peak_src, "kernel": f"k_spmv_{info['kernel_name']}<double>",
                         "traffic_source": "profiles/spmv_traffic.json (ncu --set full, dram__bytes_read+write per launch)"},
            "e2e": {"value": round(e2e_val, 2), "unit": UNIT, "h2d_bytes_per_step": 8 * nl,
                    "d2h_bytes_per_step": 2 * 8 * nl + 16},
            "gpu_launches": int(launches),
            "clocks": clk,
            "zeta_last": zeta_last,
            "cg_variant": args.cg_variant,
            "cg_variants": variants,
            "cpu_baseline": cpu,
        }
        print(json.dumps(line), flush=True)
    M.destroy()
    if d is not None:
        d.close()
    if use_dist:
        dist.destroy_process_group()


def cpu_baseline(A, shift, budget_s=15.0):
    """The oracle as it stands on a bounded sample of the same class-C workload:
    whole NAS outer iterations (after one untimed warm-up iteration, like the
    reference arm) until ~budget_s/2 of CPU work, (1) oracle/oracle_spmv.c on
    1 thread and (2) its OpenMP schedule(static) copy oracle/oracle_omp.c on
    every core of sched_getaffinity.  `value`/`cores`
    are the all-core run; `single_thread` the plain oracle."""
    import numpy as np

    import oracle
    ncores = len(os.sched_getaffinity(0))

    def timed(fn, budget):
        x = np.ones(A.n)
        fn(x)  # warm-up (page faults of the work arrays, caches)
        x[:] = 1.0
        t0 = time.perf_counter()
        steps = 0
        while True:
            fn(x)
            steps += 1
            el = time.perf_counter() - t0
            if el >= budget or steps >= 50:
                return steps, el

    half = budget_s / 2
    s1, e1 = timed(lambda x: oracle.npb_outer(A.rowptr, A.colidx, A.vals, x, 25, shift), half)
    used = [1]

    def omp(x):
        used[0] = oracle.npb_outer_omp(A.rowptr, A.colidx, A.vals, x, 25, shift, nthreads=ncores)[3]

    sN, eN = timed(omp, half)
    return {"value": round(25.0 * sN / eN, 3), "unit": UNIT, "cores": int(used[0]), "kind": "oracle",
            "sample": f"{sN} NAS CG class {CLS} outer iterations ({25 * sN} CG iterations + {sN} residual SpMVs) "
                      f"in {eN:.1f} s after 1 warm-up, oracle/oracle_omp.c (the oracle's loops, OpenMP "
                      f"schedule(static)) on {used[0]} threads",
            "single_thread": {"value": round(25.0 * s1 / e1, 3), "cores": 1,
                              "sample": f"{s1} outer iterations in {e1:.1f} s after 1 warm-up, "
                                        "oracle/oracle_spmv.c -O3 1 thread"},
            "affinity_cores": ncores, "host": _cpu_model()}


def _cpu_model():
    try:
        for ln in open("/proc/cpuinfo"):
            if ln.startswith("model name"):
                return ln.split(":", 1)[1].strip()
    except Exception:
        pass
    return None


# ---------------------------------------------------------- reference arm
def run_reference(args):
    """The reference arm of this tier is the CPU oracle, timed as it stands on
    the host cores, same metric/config; one step = one NAS outer iteration."""
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return
    import numpy as np

    import gen
    import oracle
    na, nonzer, niter, shift = gen.NPB_CLASSES[CLS]
    A = gen.makea(CLS)
    x = np.ones(A.n)
    for _ in range(args.warmup):
        oracle.npb_outer(A.rowptr, A.colidx, A.vals, x, 25, shift)
    x[:] = 1.0
    t0 = time.perf_counter()
    for _ in range(args.steps):
        oracle.npb_outer(A.rowptr, A.colidx, A.vals, x, 25, shift)
    el = time.perf_counter() - t0
    v = 25.0 * args.steps / el
    line = {
        "metric": METRIC, "value": round(v, 3), "unit": UNIT, "n_gpus": world, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": round(1e3 * el / args.steps, 2), "higher_is_better": True,
        "scaling": "strong", "vs_baseline": None, "dtype": "f64",
        "data": "synthetic (exact NPB makea class C generator, seeded)",
        "config": workload_config(A, world), "impl": "reference",
        "cpu_baseline": {"value": round(v, 3), "unit": UNIT, "cores": 1, "kind": "oracle",
                         "sample": f"{args.steps} NAS CG class {CLS} outer iterations (full workload per step), "
                                   "oracle/oracle_spmv.c -O3, 1 thread", "host": _cpu_model()},
        "e2e": {"value": round(v, 3), "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--no-cpu", action="store_true", help="skip the cpu_baseline leg")
    ap.add_argument("--cpu-budget", type=float, default=15.0)
    ap.add_argument("--cg-variant", choices=["textbook", "cgcg", "persist"],
                    default=os.environ.get("SPMV_CG_VARIANT", "cgcg"),
                    help="CG inside the NAS step: textbook (NPB conj_grad), cgcg (single reduction) or "
                         "persist (single reduction, one persistent kernel per CG solve)")
    args = ap.parse_args()
    if args.warmup < 3:
        log("warmup < 3 is not allowed by the timing rules; using 3")
        args.warmup = 3
    if args.impl == "reference":
        run_reference(args)
    else:
        run_ours(args)


if __name__ == "__main__":
    main()
