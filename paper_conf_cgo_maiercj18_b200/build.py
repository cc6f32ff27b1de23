"""Build libkperf.so (sm_100a) in-tree with nvcc.  Used by __graft_entry__.build()."""
from __future__ import annotations

import concurrent.futures as cf
import glob
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
OBJ = os.path.join(HERE, "build")
LIB = os.path.join(HERE, "libkperf.so")


def _nccl_dir() -> str:
    import importlib.util
    spec = importlib.util.find_spec("nvidia.nccl")
    if spec and spec.submodule_search_locations:
        d = list(spec.submodule_search_locations)[0]
        if os.path.exists(os.path.join(d, "lib", "libnccl.so.2")):
            return d
    return "/usr"


NVCC_FLAGS = ["-gencode", "arch=compute_100a,code=sm_100a", "-std=c++17", "-O3", "-lineinfo",
              "-Xcompiler", "-fPIC", "-Xptxas", "-v"]


def build(force: bool = False, verbose: bool = False, defines=(), out=None, csrc=None) -> str:
    csrc = csrc or CSRC  # (experiment builds: a snapshot of csrc/, see tools/ab.py)
    srcs = sorted(glob.glob(os.path.join(csrc, "*.cu")))
    deps = srcs + glob.glob(os.path.join(csrc, "*.cuh")) + [os.path.join(ROOT, "include", "kperf.h")]
    newest = max(os.path.getmtime(f) for f in deps)
    lib = out or LIB
    if not force and os.path.exists(lib) and os.path.getmtime(lib) >= newest:
        return lib
    objdir = OBJ if not defines else OBJ + "_" + "_".join(d.replace("=", "") for d in defines)
    if out:
        objdir = os.path.join(os.path.dirname(os.path.abspath(out)), "obj")
    os.makedirs(objdir, exist_ok=True)
    nccl = _nccl_dir()
    inc = ["-I", os.path.join(nccl, "include"), "-I", os.path.join(ROOT, "include")]

    def compile_one(src):
        obj = os.path.join(objdir, os.path.basename(src) + ".o")
        cmd = ["nvcc", *NVCC_FLAGS, *inc, *[f"-D{d}" for d in defines], "-c", src, "-o", obj]
        r = subprocess.run(cmd, capture_output=True, text=True)
        if r.returncode != 0:
            raise RuntimeError(f"nvcc failed for {src}:\n{r.stderr}")
        return obj, r.stderr

    with cf.ThreadPoolExecutor(max_workers=os.cpu_count() or 4) as ex:
        results = list(ex.map(compile_one, srcs))
    if verbose:
        for _, log in results:
            sys.stderr.write(log)
    objs = [o for o, _ in results]
    ncclib = os.path.join(nccl, "lib")
    cmd = ["nvcc", "-shared", "-gencode", "arch=compute_100a,code=sm_100a", "-o", lib + ".tmp", *objs,
           "-L", ncclib, "-l:libnccl.so.2", "-Xlinker", f"-rpath={ncclib}"]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"link failed:\n{r.stderr}")
    os.replace(lib + ".tmp", lib)
    return lib


if __name__ == "__main__":
    defs = [a[2:] for a in sys.argv[1:] if a.startswith("-D")]
    outs = [a[6:] for a in sys.argv[1:] if a.startswith("--out=")]
    srcd = [a[7:] for a in sys.argv[1:] if a.startswith("--csrc=")]
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv, defines=defs, out=outs[0] if outs else None,
                csrc=srcd[0] if srcd else None))
