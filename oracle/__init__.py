"""CPU oracle for the batched tridiagonal solvers -- TEST INFRASTRUCTURE ONLY.

Plain, slow, obviously-correct implementations of what Zhang, Cohen & Owens,
"Fast Tridiagonal Solvers on the GPU", PPoPP'10 (/root/reference/PAPER.md,
cited P:L<line>) computes, written in plain C (``tridiag_oracle.c``) and
wrapped here with ctypes + numpy.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (its
``cpu_baseline`` leg and ``--impl reference``) may import this package.  It
shares no code with the CUDA path (``paper_conf_ppopp_zhangco10_b200``) and
never imports it; the CUDA path never imports this.

Functions (all take (S, n) C-contiguous arrays; fp64 unless noted):

* ``thomas``      -- Thomas algorithm / GE without pivoting.
                     Pinned by: dense LAPACK gesv (n <= 16), LAPACK dgtsv,
                     manufactured solutions, POI closed form, diagonal case.
* ``cr``          -- serial textbook cyclic reduction (Fig 1).
                     Pinned by: 2log2n-1 steps, Fig 1 dataflow,
                     agreement with dgtsv, POI closed form (exact).
* ``pcr``         -- parallel cyclic reduction (Fig 2).
                     Pinned by: log2n steps, Fig 2 pairs, dgtsv.
* ``rd``          -- recursive doubling, scan form (Fig 3).
                     Pinned by: log2n+2 steps, Fig 3 scan ranges,
                     dgtsv on RD-stable input, POI closed form (exact), fp32
                     overflow onset "larger than 64".
* ``hybrid``      -- CR+PCR / CR+RD with intermediate size m (P:L572-581,
                     Fig 4).  Pinned by: Fig 4 dataflow, endpoint identities
                     (m=2 == CR, m=n == PCR/RD bitwise, Fig 17),
                     step counts (reading R13), dgtsv.
* ``rd_stone``    -- overflow-free RD in LU form (NEXT f3): rescaled 2x2
                     continuant scan + two affine scans.  Pinned by: dgtsv on
                     DD / KM (where the paper's RD overflows), dense gesv,
                     3 log2 n + 4 steps, no overflow at n = 8192.
* ``thomas_mt``   -- the paper's MT CPU solver: threads solving
                     whole systems; the timed cpu_baseline.

Every function returns x (and optionally the step count / event log of
system 0).  ``dtype=np.float32`` selects the fp32 instantiation (used only to
model the paper's fp32 behaviour, e.g. RD overflow).
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "tridiag_oracle.c")
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None

PCR, RD = 0, 1
EVENT_KINDS = {0: "cr_forward", 1: "solve2", 2: "cr_backward", 3: "pcr_update",
               4: "rd_setup", 5: "rd_scan", 6: "rd_eval"}


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (plain C99, -O2, no fast-math)."""
    with _lock:
        stale = (not os.path.exists(_LIB_PATH)
                 or os.path.getmtime(_LIB_PATH) < os.path.getmtime(_SRC))
        if force or stale:
            tmp = _LIB_PATH + f".tmp{os.getpid()}"
            cmd = ["gcc", "-std=c99", "-O2", "-fno-fast-math", "-ffp-contract=off",
                   "-fPIC", "-shared", "-pthread", "-o", tmp, _SRC, "-lm"]
            subprocess.run(cmd, check=True)
            os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def _load():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB_PATH)
        P = ctypes.c_void_p
        I64 = ctypes.c_int64
        I64P = ctypes.POINTER(ctypes.c_int64)
        for sfx in ("f64", "f32"):
            f = getattr(lib, f"oracle_thomas_{sfx}")
            f.argtypes = [P, P, P, P, P, I64, I64]
            f.restype = ctypes.c_int
            f = getattr(lib, f"oracle_thomas_mt_{sfx}")
            f.argtypes = [P, P, P, P, P, I64, I64, ctypes.c_int]
            f.restype = ctypes.c_int
            for name in ("cr", "pcr", "rd", "rd_stone"):
                f = getattr(lib, f"oracle_{name}_{sfx}")
                f.argtypes = [P, P, P, P, P, I64, I64, I64P, I64P, I64, I64P]
                f.restype = ctypes.c_int
            f = getattr(lib, f"oracle_hybrid_{sfx}")
            f.argtypes = [P, P, P, P, P, I64, I64, ctypes.c_int, I64, I64P, I64P, I64,
                          I64P]
            f.restype = ctypes.c_int
        lib.oracle_abi_version.restype = ctypes.c_int
        _lib = lib
    return _lib


def _prep(a, b, c, d, dtype):
    arrs = [np.ascontiguousarray(np.asarray(v), dtype=dtype) for v in (a, b, c, d)]
    shp = arrs[0].shape
    for v in arrs:
        if v.shape != shp:
            raise ValueError("a, b, c, d must have the same shape")
    if len(shp) == 1:
        arrs = [v.reshape(1, -1) for v in arrs]
    S, n = arrs[0].shape
    return arrs, S, n, len(shp) == 1


def _sfx(dtype):
    dt = np.dtype(dtype)
    if dt == np.float64:
        return "f64"
    if dt == np.float32:
        return "f32"
    raise ValueError(f"unsupported dtype {dt}")


def _ptr(v):
    return v.ctypes.data_as(ctypes.c_void_p)


def _finish(x, squeeze):
    return x.reshape(-1) if squeeze else x


def thomas(a, b, c, d, dtype=np.float64):
    """Thomas algorithm on every row of the (S, n) arrays."""
    lib = _load()
    (a, b, c, d), S, n, sq = _prep(a, b, c, d, dtype)
    x = np.empty_like(d)
    rc = getattr(lib, f"oracle_thomas_{_sfx(dtype)}")(
        _ptr(a), _ptr(b), _ptr(c), _ptr(d), _ptr(x), n, S)
    if rc != 0:
        raise ValueError(f"oracle_thomas failed ({rc})")
    return _finish(x, sq)


def thomas_mt(a, b, c, d, nthreads, dtype=np.float64, out=None):
    """The paper's MT solver: nthreads threads, whole systems each."""
    lib = _load()
    (a, b, c, d), S, n, sq = _prep(a, b, c, d, dtype)
    x = np.empty_like(d) if out is None else out
    rc = getattr(lib, f"oracle_thomas_mt_{_sfx(dtype)}")(
        _ptr(a), _ptr(b), _ptr(c), _ptr(d), _ptr(x), n, S, int(nthreads))
    if rc != 0:
        raise ValueError(f"oracle_thomas_mt failed ({rc})")
    return _finish(x, sq)


def _run_stepped(fname, a, b, c, d, dtype, extra, log_events, log_cap):
    lib = _load()
    (a, b, c, d), S, n, sq = _prep(a, b, c, d, dtype)
    x = np.empty_like(d)
    steps = ctypes.c_int64(0)
    log_len = ctypes.c_int64(0)
    if log_events:
        log = np.zeros((log_cap, 5), dtype=np.int64)
        log_p = log.ctypes.data_as(ctypes.POINTER(ctypes.c_int64))
    else:
        log = None
        log_p = ctypes.POINTER(ctypes.c_int64)()
    fn = getattr(lib, f"oracle_{fname}_{_sfx(dtype)}")
    rc = fn(_ptr(a), _ptr(b), _ptr(c), _ptr(d), _ptr(x), n, S, *extra,
            ctypes.byref(steps), log_p, log_cap if log_events else 0,
            ctypes.byref(log_len))
    if rc != 0:
        raise ValueError(f"oracle_{fname} rejected the arguments ({rc})")
    events = None
    if log_events:
        if log_len.value > log_cap:
            raise RuntimeError("event log truncated; raise log_cap")
        events = log[: log_len.value]
    return _finish(x, sq), steps.value, events


def cr(a, b, c, d, dtype=np.float64, log_events=False, log_cap=1 << 16):
    """Serial textbook CR.  Returns (x, steps, events|None)."""
    return _run_stepped("cr", a, b, c, d, dtype, (), log_events, log_cap)


def pcr(a, b, c, d, dtype=np.float64, log_events=False, log_cap=1 << 18):
    """PCR.  Returns (x, steps, events|None)."""
    return _run_stepped("pcr", a, b, c, d, dtype, (), log_events, log_cap)


def rd(a, b, c, d, dtype=np.float64, log_events=False, log_cap=1 << 18):
    """RD.  Returns (x, steps, events|None)."""
    return _run_stepped("rd", a, b, c, d, dtype, (), log_events, log_cap)


def rd_stone(a, b, c, d, dtype=np.float64):
    """Overflow-free RD in LU form (NEXT f3; Stone [27] as cited at P:L387-389):
    three Hillis-Steele scans -- rescaled 2x2 continuant products for the
    pivots, forward and backward affine scans.  Returns (x, steps)."""
    x, st, _ = _run_stepped("rd_stone", a, b, c, d, dtype, (), False, 0)
    return x, st


def hybrid(a, b, c, d, m, inner="pcr", dtype=np.float64, log_events=False,
           log_cap=1 << 18):
    """CR+PCR (inner='pcr') or CR+RD (inner='rd') with intermediate size m
    (Fig 4).  Returns (x, steps, events|None)."""
    code = {"pcr": PCR, "rd": RD}[inner]
    return _run_stepped("hybrid", a, b, c, d, dtype, (ctypes.c_int(code), int(m)),
                        log_events, log_cap)


def solve(algo, a, b, c, d, m=0, dtype=np.float64):
    """Dispatch by the C-ABI algorithm name: 'cr', 'pcr', 'rd', 'cr_pcr', 'cr_rd'.
    m = 0 for the hybrids means "use the caller-supplied m" is required."""
    if algo == "cr":
        return cr(a, b, c, d, dtype)[0]
    if algo == "pcr":
        return pcr(a, b, c, d, dtype)[0]
    if algo == "rd":
        return rd(a, b, c, d, dtype)[0]
    if algo == "rd_stone":
        return rd_stone(a, b, c, d, dtype)[0]
    if algo in ("cr_pcr", "cr_rd"):
        if m <= 0:
            raise ValueError("oracle.solve needs an explicit m for the hybrids")
        return hybrid(a, b, c, d, m, inner=algo[3:], dtype=dtype)[0]
    raise ValueError(algo)


def abi_version() -> int:
    return _load().oracle_abi_version()


from .metrics import normwise_error, residual_inf, tridiag_matvec  # noqa: E402,F401
