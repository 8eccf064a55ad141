"""Seeded synthetic inputs for the batched tridiagonal solvers.

This module is the ONLY code shared by the oracle side (tests, cpu_baseline)
and the CUDA side (bench, parity tests): it holds no arithmetic of the
method, only a counter-based random generator and the matrix families of
DESIGN.md "Input recipe".

Counter-based: the value of element i of system s of array k depends only on
(seed, k, global element index s*n + i), so a multi-GPU shard of systems
[s0, s0+S) generates exactly the bytes the single-GPU batch holds there
(SURVEY.md 8(e)), on any device.  The generator is written with torch int64
ops that are exact on CPU and CUDA (32-bit products are split into 16-bit
halves so no int64 product overflows), and uniforms carry 24 random bits, so
CPU and GPU generation are bitwise identical.

Families (per system, 0-based; P:L1225-1230 names the paper's two families
"diagonally dominant matrices that arise from fluid simulation" and "random
matrices with close values in all rows"; their distributions are not given,
so these are the readings R19 of DESIGN.md):

* ``dd``   a_i, c_i ~ U(-1,1); b_i = +-(|a_i| + |c_i| + U(1,2)) with a random
           sign, computed with a_0 = c_{n-1} = 0; d_i ~ U(-1,1).  The stored
           a_0 and c_{n-1} keep their random values (they are not matrix
           entries and every solver must ignore them).
* ``km``   Kass-Miller-style SPD M-matrix ("fluid simulation [20]"):
           e_j = E*U(0.5,1), j = 0..n; a_i = -e_i, c_i = -e_{i+1},
           b_i = 1 + e_i + e_{i+1}; d ~ U(-1,1).  ``E`` keyword (1 or 100).
* ``poi``  a = c = -1, b = 2; d ~ U(-1,1)   (weakly dominant, RD-stable)
* ``poi1`` a = c = -1, b = 2, d = 1: closed form x_i = (i+1)(n-i)/2.
* ``cv``   a_i, b_i, c_i ~ U(0.9,1.1); d ~ U(-1,1)  ("close values in all rows")
* ``rdw``  a_i ~ U(-0.01,0.01), b_i, c_i ~ U(0.99,1.01); d ~ U(-1,1).  Not a
           paper workload: a test family on which RD's forward recurrence
           x_{i+1} = (d_i - a_i x_{i-1} - b_i x_i) / c_i (the B_i of P:L398-401) neither
           overflows nor amplifies error at large n (characteristic roots
           ~ -b/c and ~ -a/b), so RD / CR+RD kernels can be held to the
           accuracy gates at the CTA sizes (n > 32 R).
"""
from __future__ import annotations

import torch

M32 = 0xFFFFFFFF
FAMILIES = ("dd", "km", "poi", "poi1", "cv", "rdw")
DEFAULT_SEED = 20100109  # seed = 20100109 + config index


def _mul32(x: torch.Tensor, cst: int) -> torch.Tensor:
    """(x * cst) mod 2^32 for x in [0, 2^32), exact in int64 (no overflow)."""
    lo = cst & 0xFFFF
    hi = cst >> 16
    return ((x * lo) + (((x * hi) & 0xFFFF) << 16)) & M32


def _hash32(x: torch.Tensor) -> torch.Tensor:
    """lowbias32 integer hash (C. Wellons) on int64 tensors holding uint32."""
    x = x ^ (x >> 16)
    x = _mul32(x, 0x7FEB352D)
    x = x ^ (x >> 15)
    x = _mul32(x, 0x846CA68B)
    x = x ^ (x >> 16)
    return x


def _hash32_scalar(v: int) -> int:
    v &= M32
    v ^= v >> 16
    v = (v * 0x7FEB352D) & M32
    v ^= v >> 15
    v = (v * 0x846CA68B) & M32
    v ^= v >> 16
    return v


def uniform(g: torch.Tensor, seed: int, stream: int) -> torch.Tensor:
    """U[0,1) in float64 with 24 random bits, keyed by (seed, stream, g)."""
    key = _hash32_scalar(_hash32_scalar(seed) ^ (stream * 0x9E3779B9 & M32))
    h = _hash32((g & M32) ^ key)
    h = _hash32(h ^ ((g >> 32) & M32))
    return (h >> 8).to(torch.float64) * (1.0 / (1 << 24))


def element_index(S: int, n: int, s0: int = 0, device="cpu", i0: int = 0, count=None) -> torch.Tensor:
    s = torch.arange(s0, s0 + S, dtype=torch.int64, device=device)
    i = torch.arange(i0, i0 + (n - i0 if count is None else count), dtype=torch.int64, device=device)
    return s[:, None] * n + i[None, :]


def generate(family: str, S: int, n: int, dtype=torch.float32, seed: int = DEFAULT_SEED,
             s0: int = 0, device="cpu", E: float = 1.0, poison_corners: bool = False,
             i0: int = 0, count=None):
    """Return (a, b, c, d), each an (S, n) contiguous tensor of ``dtype``.

    Values are formed in float64 and rounded once to ``dtype``; systems
    [s0, s0+S) of the global batch are produced.  ``poison_corners`` writes
    NaN into a[:, 0] and c[:, n-1], which no solver may read (reading R1).
    ``i0`` / ``count``: only equations [i0, i0+count) of each n-equation
    system, (S, count) tensors bitwise equal to those columns of the full
    systems (a huge system is generated in pieces; families dd, poi, rdw, cv).
    """
    if family not in FAMILIES:
        raise ValueError(f"unknown family {family!r}; one of {FAMILIES}")
    if S < 0 or n < 1:
        raise ValueError("need S >= 0 and n >= 1")
    cnt = n - i0 if count is None else count
    if i0 < 0 or cnt < 0 or i0 + cnt > n:
        raise ValueError("need 0 <= i0 <= i0 + count <= n")
    if (i0 != 0 or cnt != n) and (family == "km" or poison_corners):
        raise ValueError("equation ranges are supported for dd / poi / poi1 / rdw / cv without poisoning")
    g = element_index(S, n, s0, device, i0, cnt)
    f64 = torch.float64
    if family == "dd":
        a = 2.0 * uniform(g, seed, 0) - 1.0
        c = 2.0 * uniform(g, seed, 1) - 1.0
        a_in = a.clone()
        c_in = c.clone()
        if i0 == 0 and cnt > 0:
            a_in[:, 0] = 0.0
        if i0 + cnt == n and cnt > 0:
            c_in[:, cnt - 1] = 0.0
        sign = torch.where(uniform(g, seed, 3) < 0.5, -1.0, 1.0).to(f64)
        b = sign * (a_in.abs() + c_in.abs() + 1.0 + uniform(g, seed, 2))
        d = 2.0 * uniform(g, seed, 4) - 1.0
    elif family == "km":
        e_lo = E * (0.5 + 0.5 * uniform(g, seed, 0))          # e_i, i = 0..n-1
        e_last = E * (0.5 + 0.5 * uniform(g[:, n - 1:], seed, 5))  # e_n
        e_hi = torch.cat([e_lo[:, 1:], e_last], dim=1)          # e_{i+1}
        a = -e_lo
        c = -e_hi
        b = 1.0 + e_lo + e_hi
        d = 2.0 * uniform(g, seed, 4) - 1.0
    elif family in ("poi", "poi1"):
        a = torch.full(g.shape, -1.0, dtype=f64, device=device)
        c = torch.full(g.shape, -1.0, dtype=f64, device=device)
        b = torch.full(g.shape, 2.0, dtype=f64, device=device)
        if family == "poi":
            d = 2.0 * uniform(g, seed, 4) - 1.0
        else:
            d = torch.ones(g.shape, dtype=f64, device=device)
    elif family == "rdw":
        a = 0.02 * uniform(g, seed, 0) - 0.01
        b = 0.99 + 0.02 * uniform(g, seed, 2)
        c = 0.99 + 0.02 * uniform(g, seed, 1)
        d = 2.0 * uniform(g, seed, 4) - 1.0
    else:  # cv
        a = 0.9 + 0.2 * uniform(g, seed, 0)
        b = 0.9 + 0.2 * uniform(g, seed, 2)
        c = 0.9 + 0.2 * uniform(g, seed, 1)
        d = 2.0 * uniform(g, seed, 4) - 1.0
    out = [v.to(dtype).contiguous() for v in (a, b, c, d)]
    if poison_corners and n >= 1:
        out[0][:, 0] = float("nan")
        out[2][:, n - 1] = float("nan")
    return tuple(out)

