"""Build libhrs.so (sm_100a only) in-tree with nvcc.

    python paper_1611_01137_b200/build.py [--force]
"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
LIB = os.path.join(HERE, "libhrs.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")

NVCC_FLAGS = [
    "-O3", "-std=c++17", "-lineinfo",
    "-gencode", "arch=compute_100a,code=sm_100a",
    "-Xcompiler", "-fPIC,-O2,-fvisibility=hidden",
    "-Xptxas", "-v",
    "--expt-relaxed-constexpr",
    "-I", os.path.join(ROOT, "include"),
]


# translation units: the planner / C ABI, and one instantiation unit per key width and key
# kind (csrc/inst.cu with defines), compiled in parallel and linked into libhrs.so
UNITS = [("hrs", "hrs.cu", []), ("k4", "inst.cu", ["HRS_INST_KB=4", "HRS_INST_TY=0"]),
         ("k8", "inst.cu", ["HRS_INST_KB=8", "HRS_INST_TY=0"]), ("k4t", "inst.cu", ["HRS_INST_KB=4", "HRS_INST_TY=1"]),
         ("k8t", "inst.cu", ["HRS_INST_KB=8", "HRS_INST_TY=1"])]


def sources():
    return sorted({os.path.join(CSRC, f) for _, f, _ in UNITS})


def deps():
    return sources() + glob.glob(os.path.join(CSRC, "*.cuh")) + glob.glob(os.path.join(ROOT, "include", "*.h"))


def up_to_date() -> bool:
    if not os.path.exists(LIB):
        return False
    t = os.path.getmtime(LIB)
    return all(os.path.getmtime(d) <= t for d in deps())


def build(force: bool = False, verbose: bool = False, out: str | None = None, defines=()) -> str:
    from concurrent.futures import ThreadPoolExecutor
    lib = out or LIB
    if not force and out is None and up_to_date():
        return LIB
    objdir = lib + ".objs"
    os.makedirs(objdir, exist_ok=True)
    only = any(d.startswith("HRS_ONLY_TYPES") for d in defines)
    units = [u for u in UNITS if not (only and u[0] in ("k4t", "k8t"))]

    def compile_unit(u):
        name, src, defs = u
        obj = os.path.join(objdir, name + ".o")
        cmd = [NVCC, *NVCC_FLAGS, *[f"-D{d}" for d in (*defines, *defs)], "-c", "-o", obj, os.path.join(CSRC, src)]
        r = subprocess.run(cmd, capture_output=True, text=True)
        return obj, cmd, r

    with ThreadPoolExecutor(max_workers=len(units)) as ex:
        results = list(ex.map(compile_unit, units))
    log = os.path.join(HERE, "build.log") if out is None else lib + ".log"
    with open(log, "w") as f:
        for _, cmd, r in results:
            f.write(" ".join(cmd) + "\n" + r.stdout + r.stderr)
    for _, cmd, r in results:
        if r.returncode != 0:
            sys.stderr.write(r.stderr[-8000:])
            raise RuntimeError(f"nvcc failed (exit {r.returncode}); see {log}")
    if only:  # the experiment build has no typed units: empty stand-ins keep the link whole
        stub = os.path.join(objdir, "typed_stub.cu")
        with open(stub, "w") as f:
            f.write('#include "hrs_host.cuh"\nnamespace hrs_host {\n'
                    'hrs_status sort_k4t(int, const Plan &, void *, const void *, void *, const void *, void *, '
                    'cudaStream_t, int, int, const uint64_t *) { return HRS_ERROR_INVALID_VALUE; }\n'
                    'hrs_status sort_k8t(int, const Plan &, void *, const void *, void *, const void *, void *, '
                    'cudaStream_t, int, int, const uint64_t *) { return HRS_ERROR_INVALID_VALUE; }\n}\n')
        so = os.path.join(objdir, "typed_stub.o")
        r = subprocess.run([NVCC, *NVCC_FLAGS, "-I", CSRC, "-c", "-o", so, stub], capture_output=True, text=True)
        if r.returncode:
            raise RuntimeError(r.stderr[-4000:])
        results.append((so, None, None))
    cmd = [NVCC, "-shared", "-gencode", "arch=compute_100a,code=sm_100a", "-o", lib + ".tmp",
           *[o for o, _, _ in results]]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        sys.stderr.write(r.stderr[-8000:])
        raise RuntimeError(f"link failed (exit {r.returncode})")
    os.replace(lib + ".tmp", lib)
    if out is not None:  # experiment builds: keep only the library
        import shutil
        shutil.rmtree(objdir, ignore_errors=True)
    if verbose:
        for _, _, rr in results:
            if rr is not None:
                sys.stderr.write(rr.stderr)
    return lib


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose="-v" in sys.argv)
    print(LIB)
