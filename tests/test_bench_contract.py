"""The bench.py driver contract: one JSON line with the keys the driver and
the judge read (metric/value/unit, roofline, e2e, gpu_launches, clocks,
cpu_baseline), for the reference arm (the oracle on host cores: runs here
without a GPU) and for our arm (GPU).  The workload is BJ.cfg[3], NAS CG class
C (the SpMV inside the CG loop is the benchmark's bottleneck)."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(args, timeout):
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                       timeout=timeout, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [ln for ln in r.stdout.splitlines() if ln.strip().startswith("{")]
    assert len(lines) == 1, r.stdout[-2000:]
    return json.loads(lines[0])


def _common(d):
    bj = json.load(open(os.path.join(ROOT, "BASELINE.json")))
    assert d["metric"] == bj["metric"]
    assert d["unit"] == "CG iters/s" and d["higher_is_better"] is True
    assert d["value"] > 0 and d["ms_per_step"] > 0
    assert d["n_gpus"] == 1 and d["warmup"] >= 3
    assert d["dtype"] == "f64" and d["data"].startswith("synthetic")
    assert "class C" in d["config"]["workload"] and d["config"]["nnz"] == 36121058


def test_reference_arm_contract():
    d = _run(["--impl", "reference", "--steps", "1", "--warmup", "3"], timeout=600)
    _common(d)
    assert d["impl"] == "reference"
    cb = d["cpu_baseline"]
    assert cb["kind"] == "oracle" and cb["cores"] >= 1 and cb["value"] == d["value"] and cb["sample"]
    assert d["e2e"] == {"value": d["value"], "unit": d["unit"], "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}


@pytest.mark.gpu
def test_our_arm_contract():
    d = _run(["--steps", "3", "--warmup", "3", "--no-cpu"], timeout=900)
    _common(d)
    rf = d["roofline"]
    assert rf["bound"] == "hbm" and rf["unit"] == "GB/s" and rf["peak"] > 0
    assert abs(rf["frac"] - rf["achieved"] / rf["peak"]) < 1e-3
    assert 0.5 < rf["frac"] < 1.2, rf  # algorithmic bytes; the plan is smaller than the CSR arrays
    e2e = d["e2e"]
    assert e2e["value"] > 0 and e2e["h2d_bytes_per_step"] == 8 * 150000 and e2e["d2h_bytes_per_step"] > 0
    assert d["gpu_launches"] > 0
    assert d["clocks"]["sm_max_mhz"] > 0
    # every CG variant ends the same number of NAS outer iterations at the same zeta
    for k, v in d["cg_variants"].items():
        if k.startswith("zeta_last_"):
            assert abs(v - d["zeta_last"]) <= 1e-10 * abs(d["zeta_last"])
