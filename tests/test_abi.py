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


def _declared_functions(header="spmv.h"):
    txt = open(os.path.join(ROOT, "include", header)).read()
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
    for name in _declared_functions("idioms.h"):
        assert hasattr(lib, name), f"{name} declared in include/idioms.h but not exported"
    assert sorted(sp.IDIOM_EXPORTS) == _declared_functions("idioms.h")


def test_idiom_workspace_queries_and_argument_errors(sp):
    """Host-side checks of include/idioms.h (no kernel is launched)."""
    assert sp.idl_reduce_workspace(0) >= 16 and sp.idl_reduce_workspace(10**9) == sp.idl_reduce_workspace(1)
    assert sp.idl_histogram_workspace("sat_u8", 10, 1000) >= 4000
    assert sp.ep_npb_workspace() >= 16 + 12 * 8
    with pytest.raises(sp.SpmvError):
        sp.idl_histogram_workspace("count", 10, 0)
    assert sp.idl_reduce_c(7, 0, None, None, 0, None, None, 0, None) == sp.SPMV_ERR_ARG
    assert sp.idl_reduce_c(sp.SPMV_F64, 0, None, None, -1, None, None, 0, None) == sp.SPMV_ERR_ARG
    assert sp.ep_npb_c(23, 0, 1, None, None, 0, None) == sp.SPMV_ERR_ARG
    assert sp.ep_npb_c(24, (1 << 24) - 1, 2, None, None, 1 << 20, None) == sp.SPMV_ERR_ARG
    assert sp.idl_histogram_c(1, None, None, 1 << 33, 10, None, None, 1 << 20, None) == sp.SPMV_ERR_ARG


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
