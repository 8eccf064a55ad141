"""Error metrics of the oracle -- TEST INFRASTRUCTURE ONLY (see oracle/__init__.py).

* ``normwise_error``: per system e_s = max_i |x_i - xhat_i| / max_i |xhat_i|
  (reading R18: the north_star "max relative error" read normwise, because
  elementwise relative error is meaningless at near-zero components).
* ``residual_inf``: the paper's accuracy measure ||A x - d||_inf per system
  ("||Ax-b||" read as ||Ax-d||, reading R20).

Both are evaluated in fp64 on the exact upcast of their arguments.
"""
from __future__ import annotations

import numpy as np


def tridiag_matvec(a, b, c, x):
    """y = A x for every row; a_0 and c_{n-1} are not matrix entries (reading R1)."""
    a = np.asarray(a, dtype=np.float64)
    b = np.asarray(b, dtype=np.float64)
    c = np.asarray(c, dtype=np.float64)
    x = np.asarray(x, dtype=np.float64)
    y = b * x
    y[..., 1:] += a[..., 1:] * x[..., :-1]
    y[..., :-1] += c[..., :-1] * x[..., 1:]
    return y


def normwise_error(x, xhat):
    """Per-system max_i |x_i - xhat_i| / max_i |xhat_i| over the last axis.

    inf if x has a non-finite entry; 0 when x equals xhat exactly (0/0, the
    d = 0 system, reading R18). Pinned by tests/test_oracle.py
    ``test_normwise_error_*`` (hand-computed exact values)."""
    x = np.asarray(x, dtype=np.float64)
    xhat = np.asarray(xhat, dtype=np.float64)
    num = np.max(np.abs(x - xhat), axis=-1)
    den = np.max(np.abs(xhat), axis=-1)
    with np.errstate(invalid="ignore", divide="ignore"):
        e = np.where(num == 0.0, 0.0, num / den)
    bad = ~np.all(np.isfinite(x), axis=-1)
    e = np.where(bad, np.inf, e)
    return e


def residual_inf(a, b, c, d, x):
    """Per-system ||A x - d||_inf."""
    r = tridiag_matvec(a, b, c, x) - np.asarray(d, dtype=np.float64)
    return np.max(np.abs(r), axis=-1)
