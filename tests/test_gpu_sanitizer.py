"""Sanitizer tier: compute-sanitizer memcheck,
racecheck and synccheck over small invocations of every kernel family
(tools/sanitize_cases.py: the x-stationary cluster kernels with their
st.async / mbarrier / cluster-barrier protocols, the TMA rings, SELL, merge,
vector, stencil, JDS, histogram / reduction / EP, CG).  The paper's admitted
weak spot is the soundness of sparse accesses (section 6.3); a
report fails the test.  Also covered: the persistent CG kernel (grid barriers)
and the two ranks of the p2p transport, each under its own sanitizer.  The logs of the round's runs are kept in
profiles/r02_sanitizer_*.log.

Opt-in (SPMV_SANITIZE=1): compute-sanitizer was closed on this GPU pool late in
round 2 ("runs under it have left GPUs needing a reset"), so the default GPU
suite skips the tier; the committed logs are the round's evidence and
tests/test_gpu_bounds.py covers out-of-range accesses with the library's own
device-side checks (SPMV_DEBUG validation pass) instead."""
import os
import re
import shutil
import subprocess
import sys

import pytest

pytestmark = [pytest.mark.gpu,
              pytest.mark.skipif(os.environ.get("SPMV_SANITIZE") != "1",
                                 reason="compute-sanitizer tier is opt-in (SPMV_SANITIZE=1): closed on this pool")]

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SAN = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
CASES = os.path.join(ROOT, "tools", "sanitize_cases.py")


def _run(tool, cases, timeout=900):
    cmd = [SAN, "--tool", tool, "--error-exitcode", "9", "--print-limit", "20", sys.executable, CASES, *cases]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=timeout, cwd=ROOT)
    out = r.stdout + r.stderr
    if "closed on this pool" in out:
        pytest.skip("compute-sanitizer closed on this pool")
    # memcheck / synccheck: "ERROR SUMMARY: 0 errors"; racecheck: "RACECHECK SUMMARY: 0 hazards displayed (0 errors, 0 warnings)"
    clean = re.search(r"ERROR SUMMARY: 0 errors", out) or re.search(r"RACECHECK SUMMARY: 0 hazards displayed \(0 errors, 0 warnings\)", out)
    assert r.returncode == 0 and clean and "sanitize cases OK" in out, out[-4000:]


@pytest.mark.parametrize("cases", [["xplan", "xt", "cg", "persist"], ["sell", "sellsort", "merge", "vector", "xstat"],
                                   ["stencil", "jds", "idioms"]])
def test_memcheck(cases):
    _run("memcheck", cases)


@pytest.mark.parametrize("cases", [["xplan"], ["xt"], ["persist"], ["stencil", "idioms"]])
def test_racecheck(cases):
    _run("racecheck", cases, timeout=1500)


@pytest.mark.parametrize("cases", [["xplan", "xt", "persist"], ["stencil", "sell", "merge", "idioms"]])
def test_synccheck(cases):
    _run("synccheck", cases)


@pytest.mark.parametrize("tool", ["memcheck", "racecheck"])
def test_p2p_two_ranks(tool):
    """The p2p transport's two ranks (two processes on the one GPU, CUDA IPC peer
    stores and system-scope epoch flags), each rank a top-level process under
    its own compute-sanitizer, so both are instrumented."""
    import socket
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    cmd = lambda r: [SAN, "--tool", tool, "--error-exitcode", "9", "--print-limit", "20", sys.executable, CASES,  # noqa: E731
                     "p2prank", str(r), str(port)]
    ps = [subprocess.Popen(cmd(r), stdout=subprocess.PIPE, stderr=subprocess.STDOUT, text=True, cwd=ROOT) for r in (0, 1)]
    outs = []
    for p in ps:
        try:
            out, _ = p.communicate(timeout=900)
        except subprocess.TimeoutExpired:
            for q in ps:
                q.kill()
            raise
        outs.append((p.returncode, out))
    for rc, out in outs:
        clean = re.search(r"ERROR SUMMARY: 0 errors", out) or \
            re.search(r"RACECHECK SUMMARY: 0 hazards displayed \(0 errors, 0 warnings\)", out)
        assert rc == 0 and clean and "sanitize cases OK" in out, out[-4000:]
