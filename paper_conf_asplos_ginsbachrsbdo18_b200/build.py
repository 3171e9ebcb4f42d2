"""Builds libspmv_b200.so in-tree with nvcc for sm_100a (SASS, -lineinfo): one
object per csrc/*.cu unit, compiled in parallel, linked into the shared library.

NCCL is linked against the copy torch bundles (site-packages/nvidia/nccl) so a
process that also uses torch.distributed loads exactly one NCCL.
"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
LIB = os.path.join(HERE, "libspmv_b200.so")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def nccl_dir() -> str:
    import importlib.util
    spec = importlib.util.find_spec("nvidia")
    for base in (spec.submodule_search_locations if spec else []):
        d = os.path.join(base, "nccl")
        if os.path.exists(os.path.join(d, "include", "nccl.h")):
            return d
    raise RuntimeError("torch-bundled NCCL (site-packages/nvidia/nccl) not found")


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")) + glob.glob(os.path.join(CSRC, "*.cuh"))
                  + glob.glob(os.path.join(ROOT, "include", "*.h")))


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(s) > t for s in sources())


def build(force: bool = False, verbose: bool = False, flags: list[str] | None = None, out: str | None = None) -> str:
    """Compile every csrc/*.cu unit (in parallel) and link libspmv_b200.so.
    flags: extra nvcc flags (e.g. -D knobs of tools/build_variants.sh); out:
    another output path (variant builds never overwrite the product .so)."""
    lib = out or LIB
    if not force and not flags and out is None and not stale():
        return LIB
    from concurrent.futures import ThreadPoolExecutor

    nd = nccl_dir()
    nvcc = os.environ.get("NVCC", "nvcc")
    tag = f"{os.getpid()}_{abs(hash((tuple(flags or []), lib))) % 10**8}"
    objdir = os.path.join(HERE, "build", tag)
    os.makedirs(objdir, exist_ok=True)
    units = sorted(glob.glob(os.path.join(CSRC, "*.cu")))
    common = [nvcc, *ARCH, "-O3", "-lineinfo", "-std=c++17", "-Xcompiler", "-fPIC",
              "-Xptxas", "-v" if verbose else "-O3", *(flags or []),
              "-I", os.path.join(ROOT, "include"), "-I", os.path.join(nd, "include")]

    def compile_unit(u):
        o = os.path.join(objdir, os.path.basename(u) + ".o")
        r = subprocess.run(common + ["-c", u, "-o", o], capture_output=True, text=True)
        return u, o, r

    with ThreadPoolExecutor(max_workers=min(len(units), os.cpu_count() or 4)) as ex:
        results = list(ex.map(compile_unit, units))
    for u, o, r in results:
        if r.returncode != 0:
            sys.stderr.write(r.stdout + r.stderr)
            raise RuntimeError(f"nvcc failed compiling {os.path.basename(u)}")
        if verbose:
            sys.stderr.write(f"== {os.path.basename(u)}\n" + r.stderr)
    tmp = lib + f".tmp{os.getpid()}"
    cmd = [nvcc, *ARCH, "-shared", *[o for _, o, _ in results], "-o", tmp,
           "-L", os.path.join(nd, "lib"), "-l:libnccl.so.2", f"-Xlinker=-rpath={os.path.join(nd, 'lib')}",
           "-cudart", "static"]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        sys.stderr.write(r.stdout + r.stderr)
        raise RuntimeError("nvcc failed linking libspmv_b200.so")
    os.replace(tmp, lib)
    import shutil
    shutil.rmtree(objdir, ignore_errors=True)
    return lib


if __name__ == "__main__":
    # build.py [--force] [-v] [--out PATH] [nvcc flags...]
    argv = sys.argv[1:]
    out = None
    if "--out" in argv:
        i = argv.index("--out")
        out = argv[i + 1]
        del argv[i:i + 2]
    extra = [a for a in argv if a not in ("--force", "-v")]
    print(build(force="--force" in argv, verbose="-v" in argv, flags=extra or None, out=out))
