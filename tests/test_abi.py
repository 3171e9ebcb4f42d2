"""CPU tests of the C-ABI library: it loads, exports every symbol include/spmv.h
declares, and its host-side integer logic (partition, merge-path splits) agrees
bit for bit with the independent oracle implementation.  No GPU calls."""
import os
import re

import numpy as np
import pytest

import gen
import oracle

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def sp():
    from paper_conf_asplos_ginsbachrsbdo18_b200 import build
    build.build()
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    return sp


def _declared_functions():
    txt = open(os.path.join(ROOT, "include", "spmv.h")).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    names = re.findall(r"^\s*(?:const\s+)?[a-z_0-9]+\s*\*?\s*([a-z_0-9]+)\s*\(", txt, flags=re.M)
    return sorted(set(names))


def test_header_parses():
    names = _declared_functions()
    assert "spmv_csr_create" in names and "spmv_csr" in names and "cg_solve" in names
    assert "spmv_csr_destroy" in names and len(names) >= 12


def test_library_exports_every_declared_symbol(sp):
    import ctypes
    lib = ctypes.CDLL(sp.LIB_PATH)
    for name in _declared_functions():
        assert hasattr(lib, name), f"{name} declared in include/spmv.h but not exported"
    assert sorted(sp.EXPORTS) == _declared_functions()


def test_library_is_sm100a(sp):
    import subprocess
    out = subprocess.run(["cuobjdump", "--list-elf", sp.LIB_PATH], capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_status_strings(sp):
    for s in range(9):
        assert sp.spmv_status_string(s).decode().startswith("SPMV_")


def _cases():
    cases = [gen.makea("S").rowptr, gen.laplace1d(10).rowptr, np.array([0], np.int32),
             np.array([5, 5, 5, 5], np.int32), gen.powerlaw(m=4096, lmax=500.0, seed=3).rowptr]
    skew = np.zeros(100, np.int64)
    skew[50] = 10000
    skew[::7] += 1
    cases.append(np.concatenate([[0], np.cumsum(skew)]).astype(np.int32) + 17)
    return cases


@pytest.mark.parametrize("P", [1, 2, 3, 4, 7, 8, 64])
def test_partition_bitexact_vs_oracle(sp, P):
    for rp in _cases():
        assert np.array_equal(sp.spmv_csr_partition(rp, P), oracle.partition(rp, P))


@pytest.mark.parametrize("C", [1, 2, 3, 16, 1000])
def test_merge_splits_bitexact_vs_oracle(sp, C):
    for rp in _cases():
        a = sp.spmv_csr_merge_splits(rp, C)
        b = oracle.merge_path(rp, C)
        assert np.array_equal(a[0], b[0]) and np.array_equal(a[1], b[1])


def test_partition_class_c_balance(sp):
    A = gen.makea("B")
    for P in (2, 4, 8):
        b = sp.spmv_csr_partition(A.rowptr, P)
        assert np.array_equal(b, oracle.partition(A.rowptr, P))
        nz = np.diff(A.rowptr[b].astype(np.int64))
        assert nz.max() - nz.min() <= 2 * A.row_lengths().max()
