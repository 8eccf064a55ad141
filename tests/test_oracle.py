"""Pins of the CPU oracle against things other than itself (CPU only).

What pins what:
* Thomas   -- dense LAPACK gesv (n <= 16), LAPACK dgtsv, manufactured
              solutions, the POI closed form, the diagonal special case.
* CR       -- 2log2n-1 steps, Fig 1 dataflow (golden), dgtsv, POI
              closed form exactly.
* PCR      -- log2n steps, Fig 2 dataflow (golden), dgtsv.
* RD       -- log2n+2 steps, Fig 3 scan ranges (golden), dense
              solve on RD-stable input, POI closed form exactly, fp32/fp64
              overflow onset ("larger than 64").
* hybrids  -- Fig 4 dataflow (golden), step counts (reading R13), endpoint
              identities of Fig 17, dgtsv.
"""
import math
import os

import numpy as np
import pytest
import scipy.linalg
import scipy.linalg.lapack as lapack
import torch

import oracle
from paper_conf_ppopp_zhangco10_b200 import inputs

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


def gen(family, S, n, dtype=torch.float64, **kw):
    return [t.numpy() for t in inputs.generate(family, S, n, dtype, **kw)]


def dense(a, b, c):
    """Dense n x n matrix of one system (a_0, c_{n-1} are not entries)."""
    n = len(b)
    A = np.diag(np.asarray(b, np.float64))
    if n > 1:
        A += np.diag(np.asarray(a[1:], np.float64), -1)
        A += np.diag(np.asarray(c[:-1], np.float64), 1)
    return A


def gtsv(a, b, c, d):
    """LAPACK dgtsv (GE with partial pivoting; the paper's GEP is "from LAPACK")."""
    out = np.empty_like(np.asarray(d, np.float64))
    for s in range(len(b)):
        _, _, _, x, info = lapack.dgtsv(a[s, 1:].astype(np.float64), b[s].astype(np.float64),
                                        c[s, :-1].astype(np.float64), d[s].astype(np.float64))
        assert info == 0
        out[s] = x
    return out


def closed_form_poi1(n):
    """Textbook: tridiag(-1, 2, -1) x = 1 has x_i = (i+1)(n-i)/2 (0-based)."""
    i = np.arange(n, dtype=np.float64)
    return (i + 1.0) * (n - i) / 2.0


# ----------------------------------------------------------------------------- Thomas
@pytest.mark.parametrize("family", ["dd", "km", "cv", "poi"])
@pytest.mark.parametrize("n", [1, 2, 3, 5, 8, 13, 16])
def test_thomas_matches_dense_gesv(family, n):
    a, b, c, d = gen(family, 6, n, seed=11 + n)
    x = oracle.thomas(a, b, c, d)
    for s in range(6):
        ref = np.linalg.solve(dense(a[s], b[s], c[s]), d[s])
        e = np.max(np.abs(x[s] - ref)) / np.max(np.abs(ref))
        assert e <= 1e-13, (family, n, s, e)


def test_thomas_matches_dense_on_random_nonsymmetric():
    rng = np.random.default_rng(3)
    for n in range(1, 17):
        a, c = rng.uniform(-1, 1, (2, n))
        b = rng.uniform(-1, 1, n) + np.sign(rng.uniform(-1, 1, n)) * 3.0
        d = rng.uniform(-1, 1, n)
        x = oracle.thomas(a, b, c, d)
        ref = np.linalg.solve(dense(a, b, c), d)
        assert np.max(np.abs(x - ref)) <= 1e-13 * np.max(np.abs(ref))


@pytest.mark.parametrize("family,kw", [("dd", {}), ("km", {"E": 1.0}), ("km", {"E": 100.0})])
@pytest.mark.parametrize("n", [64, 512, 4096])
def test_thomas_matches_lapack_gtsv(family, kw, n):
    a, b, c, d = gen(family, 4, n, **kw)
    x = oracle.thomas(a, b, c, d)
    e = oracle.normwise_error(x, gtsv(a, b, c, d))
    assert e.max() <= 1e-12, e


@pytest.mark.parametrize("n", [2, 16, 512, 8192])
def test_thomas_manufactured_solution(n):
    a, b, c, _ = gen("dd", 3, n, seed=5)
    rng = np.random.default_rng(n)
    xs = rng.uniform(-1, 1, (3, n))
    d = oracle.tridiag_matvec(a, b, c, xs)
    x = oracle.thomas(a, b, c, d)
    # DD with margin >= 1: kappa_inf <= (max|b|+2)/1 <= 5, so error ~ 5 * few eps.
    assert oracle.normwise_error(x, xs).max() <= 1e-14


def test_thomas_closed_form_poi1():
    for n in [1, 2, 7, 64, 512]:
        a, b, c, d = gen("poi1", 1, n)
        x = oracle.thomas(a, b, c, d)
        assert np.max(np.abs(x[0] - closed_form_poi1(n))) <= 1e-12 * np.max(closed_form_poi1(n))


def test_thomas_diagonal_special_case_bitwise():
    rng = np.random.default_rng(0)
    b = rng.uniform(1, 2, (3, 32))
    d = rng.uniform(-1, 1, (3, 32))
    z = np.zeros_like(b)
    x = oracle.thomas(z, b, z, d)
    assert np.array_equal(x, d / b)


# ----------------------------------------------------------------------------- all methods
SOLVERS = {
    "cr": lambda a, b, c, d, **k: oracle.cr(a, b, c, d, **k)[0],
    "pcr": lambda a, b, c, d, **k: oracle.pcr(a, b, c, d, **k)[0],
    "cr_pcr_4": lambda a, b, c, d, **k: oracle.hybrid(a, b, c, d, min(4, d.shape[-1]), "pcr", **k)[0],
    "cr_pcr_32": lambda a, b, c, d, **k: oracle.hybrid(a, b, c, d, min(32, d.shape[-1]), "pcr", **k)[0],
}


@pytest.mark.parametrize("name", list(SOLVERS))
@pytest.mark.parametrize("family,kw", [("dd", {}), ("km", {"E": 1.0}), ("km", {"E": 100.0})])
@pytest.mark.parametrize("n", [2, 4, 8, 64, 512, 4096])
def test_cr_family_matches_lapack(name, family, kw, n):
    a, b, c, d = gen(family, 3, n, seed=100 + n, **kw)
    x = SOLVERS[name](a, b, c, d)
    e = oracle.normwise_error(x, gtsv(a, b, c, d))
    assert e.max() <= 1e-13, (name, e)


@pytest.mark.parametrize("n", [2, 4, 8, 16])
@pytest.mark.parametrize("family", ["dd", "cv", "poi"])
def test_all_methods_match_dense_small(n, family):
    """Brute force on tiny inputs: every method vs dense LAPACK gesv.  RD and
    CR+RD are held to this on the CV and POI families only: on DD they divide
    by arbitrarily small c_i and are unstable already at n = 16 (P:L1219-1224,
    DESIGN.md reading R11)."""
    a, b, c, d = gen(family, 4, n, seed=7 * n)
    ref = np.stack([np.linalg.solve(dense(a[s], b[s], c[s]), d[s]) for s in range(4)])
    outs = {"cr": oracle.cr(a, b, c, d)[0], "pcr": oracle.pcr(a, b, c, d)[0],
            "rd": oracle.rd(a, b, c, d)[0]}
    for m in [2 ** k for k in range(1, int(math.log2(n)) + 1)]:
        outs[f"cr_pcr{m}"] = oracle.hybrid(a, b, c, d, m, "pcr")[0]
        outs[f"cr_rd{m}"] = oracle.hybrid(a, b, c, d, m, "rd")[0]
    for k, x in outs.items():
        if "rd" in k and family == "dd":
            continue
        tol = 1e-12
        e = oracle.normwise_error(x, ref).max()
        assert e <= tol, (k, e)


@pytest.mark.parametrize("n", [2, 8, 64, 256, 512])
def test_rd_matches_lapack_on_poisson(n):
    """RD and CR+RD are stable on the weakly dominant POI family."""
    a, b, c, d = gen("poi", 3, n, seed=n)
    ref = gtsv(a, b, c, d)
    assert oracle.normwise_error(oracle.rd(a, b, c, d)[0], ref).max() <= 1e-10
    for m in [2, n // 2 if n > 2 else 2, n]:
        x = oracle.hybrid(a, b, c, d, m, "rd")[0]
        assert oracle.normwise_error(x, ref).max() <= 1e-10


@pytest.mark.parametrize("n", [2, 4, 64, 512])
def test_closed_form_exact_cr_rd(n):
    """POI with d = 1: CR, RD and CR+RD are exact (every intermediate is dyadic)."""
    a, b, c, d = gen("poi1", 2, n)
    ref = closed_form_poi1(n)
    assert np.array_equal(oracle.cr(a, b, c, d)[0][0], ref)
    assert np.array_equal(oracle.rd(a, b, c, d)[0][0], ref)
    for m in [2, n]:
        assert np.array_equal(oracle.hybrid(a, b, c, d, m, "rd")[0][0], ref)
    x = oracle.pcr(a, b, c, d)[0][0]
    assert np.max(np.abs(x - ref)) <= 1e-14 * ref.max()


def test_corners_are_ignored_bitwise():
    a, b, c, d = gen("dd", 3, 64)
    ap, cp = a.copy(), c.copy()
    ap[:, 0] = np.nan
    cp[:, -1] = np.nan
    for fn in (oracle.thomas, lambda *v: oracle.cr(*v)[0], lambda *v: oracle.pcr(*v)[0],
               lambda *v: oracle.rd(*v)[0], lambda *v: oracle.hybrid(*v, 8, "pcr")[0],
               lambda *v: oracle.hybrid(*v, 8, "rd")[0]):
        x1 = fn(a, b, c, d)
        x2 = fn(ap, b, cp, d)
        assert np.array_equal(x1.view(np.uint64), x2.view(np.uint64))


# ----------------------------------------------------------------------------- step counts
@pytest.mark.parametrize("L", range(1, 12))
def test_step_counts(L):
    n = 2 ** L
    a, b, c, d = gen("dd", 1, n)
    assert oracle.cr(a, b, c, d)[1] == 2 * L - 1
    assert oracle.pcr(a, b, c, d)[1] == L
    assert oracle.rd(a, b, c, d)[1] == L + 2
    for lm in range(1, L + 1):
        m = 2 ** lm
        assert oracle.hybrid(a, b, c, d, m, "pcr")[1] == 2 * L - lm      # reading R13
        assert oracle.hybrid(a, b, c, d, m, "rd")[1] == 2 * L - lm + 2   # reading R13


def test_paper_step_counts_at_512():
    """Fig 8: 8 forward + 8 backward CR steps at n = 512; Fig 15:
    CR+PCR(m=256) 1 + 7 + 1 + 1 steps; Fig 16: CR+RD(m=128) 2 + 1 + 7 + 1 + 2."""
    a, b, c, d = gen("dd", 1, 512)
    _, st, ev = oracle.cr(a, b, c, d, log_events=True)
    kinds = ev[:, 1]
    assert len(set(ev[kinds == 0, 0])) == 8 and len(set(ev[kinds == 2, 0])) == 8
    _, st, ev = oracle.hybrid(a, b, c, d, 256, "pcr", log_events=True)
    assert len(set(ev[ev[:, 1] == 3, 0])) == 7 and st == 10
    _, st, ev = oracle.hybrid(a, b, c, d, 128, "rd", log_events=True)
    assert len(set(ev[ev[:, 1] == 5, 0])) == 7 and st == 13


# ----------------------------------------------------------------------------- dataflow (golden)
def _read_golden(name):
    rows = []
    with open(os.path.join(GOLDEN, name)) as f:
        for line in f:
            line = line.split("#", 1)[0].strip()
            if line:
                rows.append(line.split())
    return rows


def _one_based(i):
    return None if i < 0 else int(i) + 1


def test_fig1_cr_dataflow():
    a, b, c, d = gen("dd", 1, 8)
    _, st, ev = oracle.cr(a, b, c, d, log_events=True)
    assert st == 5
    got = {}
    for step, kind, i, p, q in ev.tolist():
        if kind == 1:
            got.setdefault(step, ("solve", set()))[1].add((p + 1, q + 1))
        else:
            srcs = tuple(sorted(v for v in (_one_based(p), _one_based(q)) if v))
            got.setdefault(step, ({0: "update", 2: "backsub"}[kind], set()))[1].add((i + 1, srcs))
    for row in _read_golden("fig1_cr_n8.txt"):
        step, kind, items = int(row[0]), row[1], row[2:]
        if kind == "solve":
            exp = {tuple(int(v) for v in it.split(",")) for it in items}
        else:
            exp = set()
            for it in items:
                t, s = it.split(":")
                exp.add((int(t), tuple(sorted(int(v) for v in s.split(",")))))
        assert got[step] == (kind, exp), step


def test_fig2_pcr_dataflow():
    a, b, c, d = gen("dd", 1, 8)
    _, st, ev = oracle.pcr(a, b, c, d, log_events=True)
    assert st == 3
    for row in _read_golden("fig2_pcr_n8.txt"):
        step, kind, items = int(row[0]), row[1], row[2:]
        e = ev[ev[:, 0] == step]
        if kind == "solve":
            exp = {tuple(int(v) for v in it.split(",")) for it in items}
            assert {(p + 1, q + 1) for _, k, _, p, q in e.tolist() if k == 1} == exp
        else:
            exp = set()
            for it in items:
                t, s = it.split(":")
                exp.add((int(t), tuple(sorted(int(v) for v in s.split(",")))))
            got = {(i + 1, tuple(sorted(v for v in (_one_based(p), _one_based(q)) if v)))
                   for _, k, i, p, q in e.tolist() if k == 3}
            assert got == exp, step


def test_fig3_rd_scan_ranges():
    a, b, c, d = gen("poi", 1, 8)
    _, st, ev = oracle.rd(a, b, c, d, log_events=True)
    assert st == 5  # setup + 3 scan steps + evaluation
    scan = ev[ev[:, 1] == 5]
    scan_steps = sorted(set(scan[:, 0].tolist()))
    rows = _read_golden("fig3_rd_scan_n8.txt")
    assert len(scan_steps) == len(rows) == 3
    for st_id, row in zip(scan_steps, rows):
        exp = [tuple(int(v) for v in it.split(",")) for it in row[1:]]
        e = scan[scan[:, 0] == st_id]
        got = [(int(p) + 1, int(q) + 1) for _, _, i, p, q in sorted(e.tolist(), key=lambda r: r[2])]
        assert got == exp
    # Evaluation: x1 from the last product C_n, then x_i from C_{i-1}.
    evl = ev[ev[:, 1] == 6]
    assert evl[0, 2] == 0 and evl[0, 3] == 7


def test_fig4_hybrid_dataflow():
    a, b, c, d = gen("dd", 1, 8)
    rows = {r[0]: [int(v) for v in r[1:]] for r in _read_golden("fig4_hybrid_n8.txt")}
    for inner, kind in (("pcr", 3), ("rd", 6)):
        _, st, ev = oracle.hybrid(a, b, c, d, 4, inner, log_events=True)
        fwd = sorted(int(i) + 1 for i in ev[ev[:, 1] == 0, 2])
        back = sorted(int(i) + 1 for i in ev[ev[:, 1] == 2, 2])
        assert fwd == rows["forward"]
        assert back == rows["backsub"]
        # inner solver runs on the 4-equation intermediate system = e'2 e'4 e'6 e'8
        inner_idx = sorted(set(int(i) for i in ev[ev[:, 1] == kind, 2]))
        assert [2 * (j + 1) for j in inner_idx] == rows["inner"]


# ----------------------------------------------------------------------------- endpoints
@pytest.mark.parametrize("n", [2, 8, 64, 512])
def test_hybrid_endpoint_identities_bitwise(n):
    """Fig 17: the endpoints m = 2 and m = n of the hybrid sweep
    are the non-hybrid solvers.  CR (separate code path) == CR+PCR(m=2) bitwise."""
    a, b, c, d = gen("dd", 5, n, seed=n)
    x_cr = oracle.cr(a, b, c, d)[0]
    x_h = oracle.hybrid(a, b, c, d, 2, "pcr")[0]
    assert np.array_equal(x_cr.view(np.uint64), x_h.view(np.uint64))


# ----------------------------------------------------------------------------- RD overflow
def test_rd_overflow_onset_fp32_fp64():
    """"for the systems of size larger than 64, RD ... might
    overflow".  Constant rows (1, 4, 1): the scan products grow like
    (2+sqrt 3)^n, so fp32 overflows between n = 64 and 128 (predicted onset
    log(FLT_MAX)/log(2+sqrt3) = 67.4) and fp64 between 512 and 1024 (539)."""
    def rows(n, dt):
        rng = np.random.default_rng(n)
        a = np.ones((2, n), dt); c = np.ones((2, n), dt); b = 4 * np.ones((2, n), dt)
        d = rng.uniform(-1, 1, (2, n)).astype(dt)
        return a, b, c, d
    assert math.log(np.finfo(np.float32).max) / math.log(2 + math.sqrt(3)) == pytest.approx(67.4, abs=0.1)
    for n in [8, 16, 32, 64]:
        assert np.all(np.isfinite(oracle.rd(*rows(n, np.float32), dtype=np.float32)[0]))
    assert not np.all(np.isfinite(oracle.rd(*rows(128, np.float32), dtype=np.float32)[0]))
    assert np.all(np.isfinite(oracle.rd(*rows(512, np.float64))[0]))
    assert not np.all(np.isfinite(oracle.rd(*rows(1024, np.float64))[0]))


def test_fp32_instantiation_tracks_fp64():
    a, b, c, d = gen("dd", 4, 256, dtype=torch.float32)
    x64 = oracle.thomas(a, b, c, d)
    for fn in (oracle.thomas, lambda *v, dtype: oracle.cr(*v, dtype=dtype)[0]):
        x32 = fn(a, b, c, d, dtype=np.float32)
        assert oracle.normwise_error(x32, x64).max() <= 1e-5


def test_thomas_mt_equals_thomas_bitwise():
    a, b, c, d = gen("km", 37, 128, E=100.0)
    x1 = oracle.thomas(a, b, c, d)
    for t in (1, 3, 8):
        xt = oracle.thomas_mt(a, b, c, d, t)
        assert np.array_equal(x1, xt)


def test_oracle_rejects_bad_sizes():
    a, b, c, d = gen("dd", 1, 6)
    with pytest.raises(ValueError):
        oracle.cr(a, b, c, d)
    a, b, c, d = gen("dd", 1, 8)
    with pytest.raises(ValueError):
        oracle.hybrid(a, b, c, d, 3, "pcr")
    with pytest.raises(ValueError):
        oracle.hybrid(a, b, c, d, 16, "pcr")


def test_residual_metric_definition():
    a, b, c, d = gen("dd", 2, 16)
    x = oracle.thomas(a, b, c, d)
    A = dense(a[0], b[0], c[0])
    assert oracle.residual_inf(a, b, c, d, x)[0] == pytest.approx(np.max(np.abs(A @ x[0] - d[0])), abs=1e-15)
    assert np.max(scipy.linalg.norm(A @ x[0] - d[0], np.inf)) <= 1e-14


# ----------------------------------------------------------------------------- RD in LU form (NEXT f3)
@pytest.mark.parametrize("family,kw", [("dd", {}), ("km", {"E": 1.0}), ("km", {"E": 100.0}), ("poi", {})])
@pytest.mark.parametrize("n", [2, 4, 16, 64, 512, 4096])
def test_rd_stone_matches_lapack(family, kw, n):
    """The overflow-free LU-form RD solves the dominant families where the
    paper's RD overflows: vs LAPACK dgtsv."""
    a, b, c, d = gen(family, 3, n, seed=31 + n, **kw)
    x, st = oracle.rd_stone(a, b, c, d)
    tol = 1e-13 if family != "poi" else 1e-10
    assert oracle.normwise_error(x, gtsv(a, b, c, d)).max() <= tol
    assert st == 3 * int(math.log2(n)) + 4     # 3 scans + 3 setups + evaluation


def test_rd_stone_dense_small_and_no_overflow():
    for n in [2, 4, 8, 16]:
        a, b, c, d = gen("cv", 4, n, seed=n)
        ref = np.stack([np.linalg.solve(dense(a[s], b[s], c[s]), d[s]) for s in range(4)])
        assert oracle.normwise_error(oracle.rd_stone(a, b, c, d)[0], ref).max() <= 1e-12
    # (1, 4, 1) rows: the paper's RD overflows in fp32 beyond n = 64; this form does not
    n = 8192
    a = np.ones((2, n), np.float32); c = np.ones((2, n), np.float32); b = 4 * np.ones((2, n), np.float32)
    d = np.random.default_rng(0).uniform(-1, 1, (2, n)).astype(np.float32)
    x32, _ = oracle.rd_stone(a, b, c, d, dtype=np.float32)
    assert np.all(np.isfinite(x32))
    assert oracle.normwise_error(x32, oracle.thomas(a, b, c, d)).max() <= 1e-5


# ----------------------------------------------------------------------------- the error metric (R18)
# Every parity gate is decided by normwise_error, so it is pinned on values
# computed by hand (powers of two, so every expected value is exact in fp64):
# a dropped abs, a reduction over the wrong axis, a division by max|x|
# instead of max|x^|, a sum instead of a max, fp32 evaluation or a lost
# non-finite check each fails one of these.
def test_normwise_error_single_perturbation_is_delta_over_max_abs_xhat():
    xhat = np.array([1.0, -4.0, 2.0])
    x = xhat.copy()
    x[2] += 2.0 ** -10
    assert oracle.normwise_error(x, xhat) == 2.0 ** -10 / 4.0


def test_normwise_error_counts_through_abs():
    # numerator: a sign flip (x - x^ negative) must count
    assert oracle.normwise_error(np.array([-1.0, 2.0]), np.array([1.0, 2.0])) == 1.0
    # denominator: the largest |x^_i| is a negative entry
    xhat = np.array([-8.0, 1.0])
    x = np.array([-8.0, 1.0 + 2.0 ** -3])
    assert oracle.normwise_error(x, xhat) == 2.0 ** -3 / 8.0


def test_normwise_error_divides_by_the_reference_not_the_result():
    assert oracle.normwise_error(np.array([8.0, 0.0]), np.array([4.0, 0.0])) == 1.0


def test_normwise_error_is_a_max_not_a_sum():
    xhat = np.ones(4)
    x = xhat + 2.0 ** -5
    assert oracle.normwise_error(x, xhat) == 2.0 ** -5


def test_normwise_error_reduces_per_system():
    xhat = np.array([[1.0, 1.0, 1.0], [100.0, 100.0, 100.0], [-2.0, 0.5, 0.25]])
    x = xhat.copy()
    x[0, 2] += 2.0 ** -4
    x[2, 1] -= 2.0 ** -6
    e = oracle.normwise_error(x, xhat)
    assert e.shape == (3,)
    assert list(e) == [2.0 ** -4, 0.0, 2.0 ** -6 / 2.0]


def test_normwise_error_evaluates_in_fp64():
    xhat = np.array([3.0], np.float32)
    x = np.nextafter(xhat, np.float32(4.0))        # 3 + 2^-22
    assert oracle.normwise_error(x, xhat)[()] == 2.0 ** -22 / 3.0


def test_normwise_error_non_finite_is_inf():
    xhat = np.array([[1.0, 2.0], [1.0, 2.0], [1.0, 2.0]])
    x = np.array([[1.0, np.nan], [np.inf, 2.0], [1.0, 2.0]])
    assert list(oracle.normwise_error(x, xhat)) == [np.inf, np.inf, 0.0]


def test_normwise_error_exact_zero_system():
    # d = 0 gives x = x^ = 0: no error (0/0 read as 0, R18); any x != 0 is inf
    assert oracle.normwise_error(np.zeros(3), np.zeros(3)) == 0.0
    assert oracle.normwise_error(np.array([0.0, 1e-300, 0.0]), np.zeros(3)) == np.inf


def test_normwise_error_on_a_real_solve_matches_its_definition_by_hand():
    # a solve perturbed in one component of one system: exactly that system moves
    a, b, c, d = gen("dd", 5, 64, seed=77)
    xhat = oracle.thomas(a, b, c, d)
    x = xhat.copy()
    x[3, 17] += 1e-6
    e = oracle.normwise_error(x, xhat)
    assert list(e[[0, 1, 2, 4]]) == [0.0] * 4
    by_hand = abs((xhat[3, 17] + 1e-6) - xhat[3, 17]) / max(abs(v) for v in xhat[3])
    assert e[3] == by_hand
