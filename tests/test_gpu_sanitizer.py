"""Sanitizer tier: compute-sanitizer memcheck,
racecheck and synccheck over small invocations of every kernel family
(tools/sanitize_cases.py: the x-stationary cluster kernels with their
st.async / mbarrier / cluster-barrier protocols, the TMA rings, SELL, merge,
vector, stencil, JDS, histogram / reduction / EP, CG).  The paper's admitted
weak spot is the soundness of sparse accesses (section 6.3); a
report fails the test.  The logs of the round's runs are kept in
profiles/r02_sanitizer_*.log."""
import os
import re
import shutil
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SAN = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
CASES = os.path.join(ROOT, "tools", "sanitize_cases.py")


def _run(tool, cases, timeout=900):
    cmd = [SAN, "--tool", tool, "--error-exitcode", "9", "--print-limit", "20", sys.executable, CASES, *cases]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=timeout, cwd=ROOT)
    out = r.stdout + r.stderr
    # memcheck / synccheck: "ERROR SUMMARY: 0 errors"; racecheck: "RACECHECK SUMMARY: 0 hazards displayed (0 errors, 0 warnings)"
    clean = re.search(r"ERROR SUMMARY: 0 errors", out) or re.search(r"RACECHECK SUMMARY: 0 hazards displayed \(0 errors, 0 warnings\)", out)
    assert r.returncode == 0 and clean and "sanitize cases OK" in out, out[-4000:]


@pytest.mark.parametrize("cases", [["xplan", "xt", "cg"], ["sell", "sellsort", "merge", "vector", "xstat"],
                                   ["stencil", "jds", "idioms"]])
def test_memcheck(cases):
    _run("memcheck", cases)


@pytest.mark.parametrize("cases", [["xplan"], ["xt"], ["stencil", "idioms"]])
def test_racecheck(cases):
    _run("racecheck", cases, timeout=1500)


@pytest.mark.parametrize("cases", [["xplan", "xt"], ["stencil", "sell", "merge", "idioms"]])
def test_synccheck(cases):
    _run("synccheck", cases)
