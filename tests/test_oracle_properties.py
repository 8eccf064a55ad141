"""Property-based pins of the oracle (CPU, hypothesis): invariants that hold
for any input, so a plausible slip anywhere in a method (a dropped term, a
wrong neighbour index, a transposed operand) fails on some generated case.

* Row scaling by powers of two: multiplying equation i by 2^e_i (a_i, b_i,
  c_i, d_i together) is exact, and every step of Thomas, CR, PCR, RD and the
  hybrids is a ratio or product in which that factor cancels exactly (CR's
  k1 = a_i / b_lo carries 2^(e_i - e_lo), a_lo k1 carries 2^e_i, ...), so x is
  BITWISE unchanged (no overflow in the chosen exponent range).
* Every method agrees with the dense solve (numpy) on random diagonally
  dominant systems of any size the method takes, and the Thomas residual is
  at rounding level.
* Reversal: solving the reversed system (equation order and the roles of a
  and c swapped) gives the reversed solution, within rounding.
"""
import numpy as np
import pytest
from hypothesis import given, settings
from hypothesis import strategies as st

import oracle

pytestmark = pytest.mark.filterwarnings("ignore")


def dd_system(rng, S, n):
    a = rng.uniform(-1, 1, (S, n))
    c = rng.uniform(-1, 1, (S, n))
    a[:, 0] = 0.0
    c[:, -1] = 0.0
    b = (np.abs(a) + np.abs(c) + rng.uniform(1, 2, (S, n))) * rng.choice([-1.0, 1.0], (S, n))
    d = rng.uniform(-1, 1, (S, n))
    return a, b, c, d


def dense_solve(a, b, c, d):
    out = np.empty_like(d)
    for s in range(d.shape[0]):
        n = d.shape[1]
        A = np.diag(b[s])
        if n > 1:
            A += np.diag(a[s, 1:], -1) + np.diag(c[s, :-1], 1)
        out[s] = np.linalg.solve(A, d[s])
    return out


def x_of(r):
    """The solution of an oracle call (the step-counting models also return
    their step count and event log)."""
    return r[0] if isinstance(r, tuple) else r


def methods(n):
    out = [("thomas", lambda a, b, c, d: oracle.thomas(a, b, c, d))]
    if n >= 2 and n & (n - 1) == 0:
        out += [("cr", lambda a, b, c, d: x_of(oracle.cr(a, b, c, d))),
                ("pcr", lambda a, b, c, d: x_of(oracle.pcr(a, b, c, d)))]
        for m in (2, max(2, n // 4), n):
            if m <= n:
                out.append((f"cr_pcr_m{m}",
                            lambda a, b, c, d, m=m: x_of(oracle.hybrid(a, b, c, d, m, inner="pcr"))))
    return out


@settings(max_examples=40, deadline=None)
@given(log2n=st.integers(1, 7), seed=st.integers(0, 2**31 - 1), S=st.integers(1, 3))
def test_power_of_two_row_scaling_is_bitwise_invisible(log2n, seed, S):
    n = 1 << log2n
    rng = np.random.default_rng(seed)
    a, b, c, d = dd_system(rng, S, n)
    e = np.ldexp(1.0, rng.integers(-40, 41, (S, n)))
    for name, f in methods(n):
        x0 = f(a, b, c, d)
        x1 = f(a * e, b * e, c * e, d * e)
        assert np.array_equal(x0, x1), name


@settings(max_examples=40, deadline=None)
@given(log2n=st.integers(1, 6), seed=st.integers(0, 2**31 - 1))
def test_rd_row_scaling_is_bitwise_invisible(log2n, seed):
    """RD (and CR+RD) on the RD-stable weakly dominant family (|b|, |c| ~ 1,
    small a), where its matrices stay finite."""
    n = 1 << log2n
    rng = np.random.default_rng(seed)
    a = rng.uniform(-0.01, 0.01, (2, n))
    b = rng.uniform(0.99, 1.01, (2, n))
    c = rng.uniform(0.99, 1.01, (2, n))
    d = rng.uniform(-1, 1, (2, n))
    e = np.ldexp(1.0, rng.integers(-30, 31, (2, n)))
    for name, f in [("rd", lambda a, b, c, d: x_of(oracle.rd(a, b, c, d)))] + [
            (f"cr_rd_m{m}", lambda a, b, c, d, m=m: x_of(oracle.hybrid(a, b, c, d, m, inner="rd")))
            for m in (2, max(2, n // 2)) if m <= n]:
        x0 = f(a, b, c, d)
        x1 = f(a * e, b * e, c * e, d * e)
        assert np.array_equal(x0, x1), name


@settings(max_examples=60, deadline=None)
@given(n=st.integers(1, 48), seed=st.integers(0, 2**31 - 1))
def test_every_method_matches_the_dense_solve(n, seed):
    rng = np.random.default_rng(seed)
    a, b, c, d = dd_system(rng, 2, n)
    ref = dense_solve(a, b, c, d)
    for name, f in methods(n):
        x = f(a, b, c, d)
        err = np.max(np.abs(x - ref)) / max(np.max(np.abs(ref)), 1e-300)
        assert err <= 1e-13, (name, n, err)
    r = oracle.residual_inf(a, b, c, d, oracle.thomas(a, b, c, d))
    assert np.max(r) <= 1e-14 * max(1.0, float(np.max(np.abs(d)))) * 8, np.max(r)


@settings(max_examples=40, deadline=None)
@given(log2n=st.integers(1, 7), seed=st.integers(0, 2**31 - 1))
def test_reversed_system_gives_reversed_solution(log2n, seed):
    n = 1 << log2n
    rng = np.random.default_rng(seed)
    a, b, c, d = dd_system(rng, 2, n)
    # equation i of the reversed system is equation n-1-i with x reversed:
    # a' = c reversed, c' = a reversed (the outer entries stay outside)
    ar, br, cr_, dr = c[:, ::-1].copy(), b[:, ::-1].copy(), a[:, ::-1].copy(), d[:, ::-1].copy()
    for name, f in methods(n):
        x = f(a, b, c, d)
        xr = f(ar, br, cr_, dr)
        err = np.max(np.abs(xr[:, ::-1] - x)) / np.max(np.abs(x))
        assert err <= 1e-13, (name, err)
