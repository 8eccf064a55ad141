"""Build libtridiag.so in-tree with nvcc for sm_100a (no JIT cache: the .so
travels with the repository snapshot to the GPU box)."""
from __future__ import annotations

import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
INCLUDE = os.path.join(ROOT, "include")
LIB = os.path.join(PKG, "libtridiag.so")
SOURCES = ["tridiag_api.cu", "inst_f32_pcr.cu", "inst_f32_rd.cu", "inst_f64_pcr.cu",
           "inst_f64_rd.cu", "inst_f32_stone.cu", "inst_f64_stone.cu", "inst_large.cu", "inst_col.cu",
           "inst_paper.cu"]
DEPS = SOURCES + ["tridiag_device.cuh", "tridiag_kernels.cuh", "tridiag_tma.cuh",
                  "tridiag_ileave.cuh", "tridiag_large.cuh", "tridiag_colpass.cuh", "tridiag_paper.cuh", "launch.cuh",
                  "host_common.h"]

NVCC_FLAGS = [
    "-gencode", "arch=compute_100a,code=sm_100a",
    "-O3", "-lineinfo", "-std=c++17",
    "-Xcompiler", "-fPIC", "-shared",
    "-Xptxas", "-v",
    # IEEE division / reciprocal and no flush-to-zero (reading R17);
    # FMA contraction allowed (reading R16).
    "-prec-div=true", "-ftz=false", "-fmad=true",
]


def nvcc() -> str:
    for cand in (os.environ.get("NVCC"), "/usr/local/cuda/bin/nvcc", "nvcc"):
        if cand and (os.path.isabs(cand) and os.path.exists(cand) or not os.path.isabs(cand)):
            return cand
    return "nvcc"


def _stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    files = [os.path.join(CSRC, f) for f in DEPS] + [os.path.join(INCLUDE, "tridiag.h")]
    return any(os.path.getmtime(f) > t for f in files)


def build(force: bool = False, verbose: bool = False) -> str:
    """Compile libtridiag.so if missing or older than its sources: one nvcc per
    translation unit (in parallel), then one link."""
    if not force and not _stale() and not os.environ.get("TRIDIAG_BUILD_OUT"):
        return LIB
    from concurrent.futures import ThreadPoolExecutor
    import tempfile
    objdir = tempfile.mkdtemp(prefix="tridiag_build_")
    compile_flags = [f for f in NVCC_FLAGS if f != "-shared"]
    # development A/B builds only (tools/build_ab.sh): extra -D flags and another
    # output path; the product build sets neither
    compile_flags += os.environ.get("TRIDIAG_NVCC_DEFINES", "").split()
    out = os.environ.get("TRIDIAG_BUILD_OUT") or LIB

    def compile_one(src):
        obj = os.path.join(objdir, os.path.splitext(src)[0] + ".o")
        cmd = [nvcc(), *compile_flags, "-dc" if False else "-c", "-I", INCLUDE, "-I", CSRC,
               "-o", obj, os.path.join(CSRC, src)]
        res = subprocess.run(cmd, capture_output=True, text=True)
        return src, obj, res

    with ThreadPoolExecutor(max_workers=min(len(SOURCES), os.cpu_count() or 4)) as ex:
        results = list(ex.map(compile_one, SOURCES))
    log_txt = ""
    for src, obj, res in results:
        log_txt += f"==== {src}\n" + res.stderr
        if res.returncode != 0:
            sys.stderr.write(res.stdout + res.stderr)
            raise RuntimeError(f"nvcc failed building {src}")
    tmp = out + f".tmp{os.getpid()}"
    link = [nvcc(), "-gencode", "arch=compute_100a,code=sm_100a", "-shared", "-Xcompiler", "-fPIC",
            "-o", tmp, *[obj for _, obj, _ in results]]
    res = subprocess.run(link, capture_output=True, text=True)
    if res.returncode != 0:
        sys.stderr.write(res.stdout + res.stderr)
        raise RuntimeError("nvcc link of libtridiag.so failed")
    with open(os.path.join(PKG, "csrc", "ptxas_last_build.txt"), "w") as f:
        f.write(log_txt)
    if verbose:
        sys.stderr.write(log_txt)
    os.replace(tmp, out)
    return out


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv))
