"""Thin Python binding of libtridiag.so (include/tridiag.h).

Argument marshalling only: every step of the solve runs in the library's
sm_100a kernels.  torch supplies device memory and the current stream.  If
the shared library is missing or fails to load, every call raises -- there
is no CPU fallback.
"""
from __future__ import annotations

import ctypes
import os
import threading

import torch

from . import build as _build

ALGOS = {"cr": 0, "pcr": 1, "rd": 2, "cr_pcr": 3, "cr_rd": 4, "rd_stone": 5}
DTYPES = {torch.float32: 0, torch.float64: 1}
HYBRIDS = ("cr_pcr", "cr_rd")

_lock = threading.Lock()
_lib = None


class TridiagError(RuntimeError):
    """CUDA-side failure reported by libtridiag (positive status)."""


def lib_path() -> str:
    # TRIDIAG_LIB_AB: another in-tree build of the same library under <repo>/ab/
    # (tools/build_ab.sh), for A/B timing of two builds on one box
    # (tools/ab_bench.sh); never set by the product, and nothing outside ab/
    # is accepted
    ab = os.environ.get("TRIDIAG_LIB_AB")
    if not ab:
        return _build.LIB
    ab_dir = os.path.realpath(os.path.join(_build.ROOT, "ab"))
    p = os.path.realpath(ab if os.path.isabs(ab) else os.path.join(_build.ROOT, ab))
    if os.path.dirname(p) != ab_dir:
        raise RuntimeError(f"TRIDIAG_LIB_AB must name a build under {ab_dir}")
    return p


def load(build_if_missing: bool = True) -> ctypes.CDLL:
    """Load libtridiag.so (building it in-tree first if it is missing/stale)."""
    global _lib
    with _lock:
        if _lib is not None:
            return _lib
        if build_if_missing and not os.environ.get("TRIDIAG_LIB_AB"):
            try:
                _build.build()
            except (OSError, RuntimeError) as e:  # no nvcc on this machine
                if not os.path.exists(_build.LIB):
                    raise RuntimeError(f"libtridiag.so is missing and could not be built: {e}")
        if not os.path.exists(lib_path()):
            raise RuntimeError(f"libtridiag.so not found at {lib_path()}; run __graft_entry__.build()")
        L = ctypes.CDLL(lib_path())
        P, I64, I = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int
        L.tridiag_solve_batched.argtypes = [P, P, P, P, P, I64, I64, I, I, I, P]
        L.tridiag_solve_batched.restype = I
        L.tridiag_solve_batched_strided.argtypes = [P, P, P, P, P, I64, I64, I64, I64, I, I, I, P]
        L.tridiag_solve_batched_strided.restype = I
        L.tridiag_solve_batched_host.argtypes = [P, P, P, P, P, I64, I64, I, I, I, P,
                                                 ctypes.c_size_t, I64]
        L.tridiag_solve_batched_host.restype = I
        L.tridiag_host_workspace_bytes.argtypes = [I64, I, I64]
        L.tridiag_host_workspace_bytes.restype = ctypes.c_size_t
        L.tridiag_status_string.argtypes = [I]
        L.tridiag_status_string.restype = ctypes.c_char_p
        L.tridiag_max_n.argtypes = [I, I]
        L.tridiag_max_n.restype = I64
        L.tridiag_max_switch_level.argtypes = [I, I, I64]
        L.tridiag_max_switch_level.restype = I64
        L.tridiag_auto_switch_level.argtypes = [I64, I, I]
        L.tridiag_auto_switch_level.restype = I
        L.tridiag_paper_cr.argtypes = [P, P, P, P, P, I64, I64, I, I, P]
        L.tridiag_paper_cr.restype = I
        L.tridiag_last_kernel_name.argtypes = [I]
        L.tridiag_last_kernel_name.restype = ctypes.c_char_p
        L.tridiag_reload_knobs.argtypes = []
        L.tridiag_reload_knobs.restype = None
        L.tridiag_abi_version.argtypes = []
        L.tridiag_abi_version.restype = I
        L.tridiag_last_launch_count.argtypes = []
        L.tridiag_last_launch_count.restype = I
        L.tridiag_phase_stamps.argtypes = [P, I64]
        L.tridiag_phase_stamps.restype = I64
        L.tridiag_phase_stamps_of.argtypes = [I, P, I64]
        L.tridiag_phase_stamps_of.restype = I64
        L.tridiag_solve_batched_large.argtypes = [P, P, P, P, P, I64, I64, I, I, I, I64, P, I64, P]
        L.tridiag_solve_batched_large.restype = I
        L.tridiag_large_workspace_bytes.argtypes = [I64, I64, I, I, I, I64]
        L.tridiag_large_workspace_bytes.restype = I64
        L.tridiag_max_n_large.argtypes = [I, I]
        L.tridiag_max_n_large.restype = I64
        L.tridiag_large_chunk.argtypes = [I]
        L.tridiag_large_chunk.restype = I64
        L.tridiag_solve_batched_strided_large.argtypes = [P, P, P, P, P, I64, I64, I64, I64, I, I,
                                                          I, I64, P, I64, P]
        L.tridiag_solve_batched_strided_large.restype = I
        L.tridiag_strided_large_workspace_bytes.argtypes = [I64, I64, I64, I64, I, I, I, I64]
        L.tridiag_strided_large_workspace_bytes.restype = I64
        L.tridiag_column_chunk.argtypes = [I]
        L.tridiag_column_chunk.restype = I64
        _lib = L
        return L


def _dtype_code(dtype) -> int:
    if isinstance(dtype, int):
        return dtype
    if dtype in DTYPES:
        return DTYPES[dtype]
    s = str(dtype).replace("torch.", "")
    return {"float32": 0, "f32": 0, "float64": 1, "f64": 1}[s]


def _algo_code(algo) -> int:
    return algo if isinstance(algo, int) else ALGOS[algo]


def status_string(status: int) -> str:
    return load().tridiag_status_string(int(status)).decode()


def check(status: int) -> None:
    if status < 0:
        raise ValueError(f"tridiag: {status_string(status)} (status {status})")
    if status > 0:
        raise TridiagError(f"tridiag: CUDA error {status}: {status_string(status)}")


_MAX_N = {}  # (dtype code, algo code) -> tridiag_max_n (immutable per build)

# torch's own fast accessors (what torch.cuda.current_stream / current_device
# call underneath), with the public API as the fallback
_current_device = getattr(torch._C, "_cuda_getDevice", None) or torch.cuda.current_device
_raw_stream = getattr(torch._C, "_cuda_getCurrentRawStream", None)


def _current_raw_stream(index: int) -> int:
    if _raw_stream is not None:
        return _raw_stream(index)
    return torch.cuda.current_stream(index).cuda_stream


def max_n(dtype, algo) -> int:
    key = (_dtype_code(dtype), _algo_code(algo))
    v = _MAX_N.get(key)
    if v is None:
        v = _MAX_N[key] = int(load().tridiag_max_n(*key))
    return v


def max_n_large(dtype, algo) -> int:
    return int(load().tridiag_max_n_large(_dtype_code(dtype), _algo_code(algo)))


def large_chunk(dtype) -> int:
    return int(load().tridiag_large_chunk(_dtype_code(dtype)))


def large_workspace_bytes(n: int, num_systems: int, dtype, algo, switch_level=0,
                          bottom_n=0) -> int:
    v = int(load().tridiag_large_workspace_bytes(int(n), int(num_systems), _dtype_code(dtype),
                                                 _algo_code(algo), int(switch_level),
                                                 int(bottom_n)))
    if v < 0:
        raise ValueError("tridiag: invalid arguments for the large-n path")
    return v


def column_chunk(dtype) -> int:
    return int(load().tridiag_column_chunk(_dtype_code(dtype)))


def strided_large_workspace_bytes(n: int, num_systems: int, elem_stride: int, sys_stride: int,
                                  dtype, algo, switch_level=0, bottom_n=0) -> int:
    v = int(load().tridiag_strided_large_workspace_bytes(
        int(n), int(num_systems), int(elem_stride), int(sys_stride), _dtype_code(dtype),
        _algo_code(algo), int(switch_level), int(bottom_n)))
    if v < 0:
        raise ValueError("tridiag: invalid arguments for the strided large path")
    return v


def _pad_n(n: int) -> int:
    return 1 << max(1, (int(n) - 1).bit_length())


def max_switch_level(dtype, algo, n: int) -> int:
    return int(load().tridiag_max_switch_level(_dtype_code(dtype), _algo_code(algo), int(n)))


def auto_switch_level(n: int, dtype, algo) -> int:
    return int(load().tridiag_auto_switch_level(int(n), _dtype_code(dtype), _algo_code(algo)))


def paper_cr(a, b, c, d, x=None, mode=0, stream=None):
    """BASELINE ONLY (tridiag_paper_cr): the paper's GT200 CR schedule, one
    CTA per system in shared memory.  mode 1 = the stride-one timing control
    (meaningless x).  Contiguous (S, n) CUDA tensors."""
    if x is None:
        x = torch.empty_like(d)
    _check_tensors([a, b, c, d, x], "cuda")
    S, n = d.shape
    raw = _current_raw_stream(d.device.index) if stream is None else stream.cuda_stream
    with torch.cuda.device(d.device):
        st = load().tridiag_paper_cr(a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                     x.data_ptr(), n, S, _dtype_code(d.dtype), int(mode), raw)
    check(st)
    return x


def last_kernel_names() -> list:
    """Mangled names of the kernels the last call on this thread launched."""
    L = load()
    out = []
    for i in range(min(last_launch_count(), 16)):
        v = L.tridiag_last_kernel_name(i)
        if v is None:
            break
        out.append(v.decode())
    return out


def reload_knobs() -> None:
    """Re-read the TRIDIAG_* tuning knobs (diagnostic; tridiag_reload_knobs)."""
    load().tridiag_reload_knobs()


def abi_version() -> int:
    return int(load().tridiag_abi_version())


def last_launch_count() -> int:
    return int(load().tridiag_last_launch_count())


def phase_stamps(cap: int = 1 << 20, launch: int = -1, width: int = 8):
    """Per-phase clock64() stamps (TRIDIAG_PHASE_STAMPS=1 only) of the last
    launch of the last call (launch=-1) or of launch `launch` of it, as a
    (rows, width) int64 tensor; empty when inactive."""
    buf = torch.zeros(cap, dtype=torch.int64)
    L = load()
    if launch < 0:
        n = int(L.tridiag_phase_stamps(buf.data_ptr(), cap))
    else:
        n = int(L.tridiag_phase_stamps_of(int(launch), buf.data_ptr(), cap))
    return buf[: n - n % width].view(-1, width)


def solve_batched_raw(a_ptr, b_ptr, c_ptr, d_ptr, x_ptr, n, num_systems, dtype, algo,
                      switch_level=0, stream=0) -> int:
    """Direct C-ABI call with integer pointers; returns the status code."""
    L = load()
    return int(L.tridiag_solve_batched(a_ptr, b_ptr, c_ptr, d_ptr, x_ptr, int(n),
                                       int(num_systems), _dtype_code(dtype), _algo_code(algo),
                                       int(switch_level), stream))


def solve_batched_strided_raw(a_ptr, b_ptr, c_ptr, d_ptr, x_ptr, n, num_systems, elem_stride,
                              sys_stride, dtype, algo, switch_level=0, stream=0) -> int:
    """Direct C-ABI call of tridiag_solve_batched_strided; returns the status."""
    L = load()
    return int(L.tridiag_solve_batched_strided(a_ptr, b_ptr, c_ptr, d_ptr, x_ptr, int(n),
                                               int(num_systems), int(elem_stride),
                                               int(sys_stride), _dtype_code(dtype),
                                               _algo_code(algo), int(switch_level), stream))


def _check_tensors(ts, device_kind, same_strides=False):
    t0 = ts[0]
    if t0.dim() != 2:
        raise ValueError("tensors must be (num_systems, n)")
    for t in ts:
        if t.shape != t0.shape or t.dtype != t0.dtype:
            raise ValueError("a, b, c, d, x must share shape and dtype")
        if same_strides:
            if t.stride() != t0.stride():
                raise ValueError("a, b, c, d, x must share strides")
        elif not t.is_contiguous():
            raise ValueError("tensors must be contiguous")
        if device_kind == "cuda" and (not t.is_cuda or t.device != t0.device):
            raise ValueError("tensors must be on the same CUDA device")
        if device_kind == "cpu" and t.is_cuda:
            raise ValueError("host API takes CPU tensors")
    if t0.dtype not in DTYPES:
        raise ValueError("dtype must be float32 or float64")


def solve_batched(a, b, c, d, x=None, algo="cr_pcr", switch_level=0, stream=None):
    """Solve the (S, n) batch a_i x_{i-1} + b_i x_i + c_i x_{i+1} = d_i on the GPU.

    a, b, c, d: CUDA tensors (float32/float64) of shape (S, n) -- row s is
    system s -- with identical strides: contiguous, pitched rows, or
    transposed views such as ``grid.T`` for the column sweep of ADI
    (tridiag_solve_batched_strided).
    x: output tensor with the same strides (may be d itself); allocated if None.
    algo: 'cr' | 'pcr' | 'rd' | 'cr_pcr' | 'cr_rd' (the paper's five) | 'rd_stone'
      (overflow-free LU-form recursive doubling, n <= 512 fp32 / 256 fp64).
    switch_level: intermediate size m of the hybrids (0 = tuned table).
    Enqueued asynchronously on ``stream`` (default: torch's current stream).
    """
    if x is None:
        x = torch.empty_strided(d.shape, d.stride(), dtype=d.dtype, device=d.device)
    # cheap common-case validation (the per-call host cost matters for small
    # batches); anything unusual goes through the full check for its message
    shape, strides, dt, dev = d.shape, d.stride(), d.dtype, d.device
    if (len(shape) != 2 or not d.is_cuda or dt not in DTYPES
            or any(t.shape != shape or t.dtype != dt or t.stride() != strides or t.device != dev
                   for t in (a, b, c, x))):
        _check_tensors([a, b, c, d, x], "cuda", same_strides=True)
    S, n = shape
    ss, es = strides
    contiguous = es == 1 and (ss == n or S <= 1)
    if contiguous:
        pn = _pad_n(n)
        if pn > max_n(dt, algo) and pn <= max_n_large(dt, algo):
            return solve_batched_large(a, b, c, d, x, algo=algo, switch_level=switch_level,
                                       stream=stream)
    else:
        # pitched rows / interleaved columns: the workspace entry point (column
        # or row passes where the on-chip strided kernels would be slow or
        # too small; none needed otherwise)
        return solve_batched_strided_large(a, b, c, d, x, algo=algo, switch_level=switch_level,
                                           stream=stream)
    L = _lib if _lib is not None else load()
    if dev.index != _current_device():
        with torch.cuda.device(dev):
            return solve_batched(a, b, c, d, x=x, algo=algo, switch_level=switch_level, stream=stream)
    raw = _current_raw_stream(dev.index) if stream is None else stream.cuda_stream
    st = L.tridiag_solve_batched(a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                 x.data_ptr(), n, S, DTYPES[dt], _algo_code(algo),
                                 int(switch_level), raw)
    if st != 0:
        check(st)
    return x


def solve_batched_strided_large(a, b, c, d, x=None, algo="cr_pcr", switch_level=0, bottom_n=0,
                                workspace=None, stream=None):
    """tridiag_solve_batched_strided_large: (S, n) CUDA tensor views with
    identical strides (pitched rows, or interleaved columns such as
    ``grid.T``).  Interleaved systems with n > 32 R go through column CR
    passes with a workspace (allocated from torch's caching allocator on
    ``stream`` if None); rows beyond one CTA through the large-n row passes."""
    if x is None:
        x = torch.empty_strided(d.shape, d.stride(), dtype=d.dtype, device=d.device)
    _check_tensors([a, b, c, d, x], "cuda", same_strides=True)
    S, n = d.shape
    ss, es = d.stride()
    ss, es = max(ss, 1), max(es, 1)
    if stream is None:
        stream = torch.cuda.current_stream(d.device)
    try:
        need = strided_large_workspace_bytes(n, S, es, ss, d.dtype, algo, switch_level, bottom_n)
    except ValueError:
        need = 0  # the call itself reports the precise status
    if workspace is None and need > 0:
        with torch.cuda.device(d.device), torch.cuda.stream(stream):
            workspace = torch.empty(need, dtype=torch.uint8, device=d.device)
    wp = workspace.data_ptr() if workspace is not None else None
    wn = workspace.numel() if workspace is not None else 0
    with torch.cuda.device(d.device):
        st = load().tridiag_solve_batched_strided_large(
            a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(), x.data_ptr(), n, S, es, ss,
            _dtype_code(d.dtype), _algo_code(algo), int(switch_level), int(bottom_n), wp, wn,
            stream.cuda_stream)
    check(st)
    return x


def solve_batched_large(a, b, c, d, x=None, algo="cr_pcr", switch_level=0, bottom_n=0,
                        workspace=None, stream=None):
    """tridiag_solve_batched_large: CR / CR+PCR / CR+RD for n beyond one CTA
    (up to 2^30), contiguous (S, n) CUDA tensors.  Reduction passes of
    log2 R CR levels shrink each system until it has <= bottom_n equations
    (0 = tridiag_max_n), the on-chip kernels solve it, expansion passes
    back-substitute.  ``workspace``: CUDA uint8 tensor of at least
    large_workspace_bytes(...) bytes, allocated from torch's caching allocator
    if None (it is used on ``stream``)."""
    if x is None:
        x = torch.empty_like(d)
    _check_tensors([a, b, c, d, x], "cuda")
    S, n = d.shape
    if stream is None:
        stream = torch.cuda.current_stream(d.device)
    need = large_workspace_bytes(n, S, d.dtype, algo, switch_level, bottom_n)
    if workspace is None:
        with torch.cuda.device(d.device), torch.cuda.stream(stream):
            workspace = torch.empty(max(need, 1), dtype=torch.uint8, device=d.device)
    with torch.cuda.device(d.device):
        st = load().tridiag_solve_batched_large(
            a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(), x.data_ptr(), n, S,
            _dtype_code(d.dtype), _algo_code(algo), int(switch_level), int(bottom_n),
            workspace.data_ptr(), workspace.numel(), stream.cuda_stream)
    check(st)
    return x


def host_workspace_bytes(n: int, dtype, chunk_systems: int = 0) -> int:
    return int(load().tridiag_host_workspace_bytes(int(n), _dtype_code(dtype), int(chunk_systems)))


def solve_batched_host(a, b, c, d, x=None, algo="cr_pcr", switch_level=0, chunk_systems=0,
                       workspace=None, device=None):
    """Solve a batch held in HOST memory (pinned CPU tensors for full speed).

    The library pipelines chunks over three streams (H2D, solve, D2H overlap)
    and returns when x is written.  ``workspace`` is a CUDA uint8 tensor of at
    least host_workspace_bytes(n, dtype, chunk_systems) bytes (allocated if None).
    """
    if x is None:
        x = torch.empty_like(d)
    _check_tensors([a, b, c, d, x], "cpu")
    S, n = d.shape
    dev = torch.device("cuda", torch.cuda.current_device()) if device is None else torch.device(device)
    need = host_workspace_bytes(n, d.dtype, chunk_systems)
    if workspace is None:
        workspace = torch.empty(need, dtype=torch.uint8, device=dev)
    # the library's internal streams write the workspace: work still queued on
    # the current (possibly non-blocking) stream must not be using it
    torch.cuda.current_stream(workspace.device).synchronize()
    with torch.cuda.device(workspace.device):
        st = load().tridiag_solve_batched_host(
            a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(), x.data_ptr(), n, S,
            _dtype_code(d.dtype), _algo_code(algo), int(switch_level), workspace.data_ptr(),
            workspace.numel(), int(chunk_systems))
    check(st)
    return x
