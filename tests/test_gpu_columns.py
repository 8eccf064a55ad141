"""GPU parity of the interleaved-layout column passes (the ADI column sweep,
NEXT f1 + f2 of SURVEY.md 8(f); ADI: P:L105-107; CR passes:
P:L280-300).

Columns of a row-major (n, S) grid are S systems with element stride S and
system stride 1.  For n > 32 R the strided-large entry point reduces them with
column CR passes (the last one writing the reduced systems transposed, as
contiguous rows), solves those with the row kernels and expands.  Every CR update is the same correctly rounded operation sequence as
the contiguous kernels', so:

* bitwise: x equals the contiguous solve of the transposed data (CR, CR+PCR
  at the default and explicit m; CR+RD within tolerance, R25), for ragged S (partial 32-system
  groups), ragged n, several passes (bottom_n), in place x == d;
* tolerances: G1/G2 against fp64 Thomas on DD, CR+RD on the RD-stable rdw
  family; columns longer than tridiag_max_n against the row large-n path.
"""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs

pytestmark = pytest.mark.gpu

TOL = {torch.float32: 1e-4, torch.float64: 1e-10}


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    td.load()


def gen(family, S, n, dtype, seed=inputs.DEFAULT_SEED):
    return inputs.generate(family, S, n, dtype, seed=seed, device="cuda")


def as_columns(ts):
    """(S, n) contiguous -> (S, n) views of (n, S) row-major grids (strides (1, S))."""
    return [t.t().contiguous().t() for t in ts]


def err(a, b, c, d, x):
    h = [t.detach().cpu().numpy() for t in (a, b, c, d)]
    return oracle.normwise_error(x.detach().contiguous().cpu().numpy(), oracle.thomas(*h))


def cols_solve(views, algo, m=0, bottom=0, x=None):
    x = td.solve_batched_strided_large(*views, x=x, algo=algo, switch_level=m, bottom_n=bottom)
    torch.cuda.synchronize()
    return x


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_column_passes_bitwise_equal_contiguous(dtype):
    mx = td.max_n(dtype, "cr")
    for n, S in ((1024, 64), (2048, 33), (mx, 40), (mx // 2, 3), (4096 if dtype == torch.float32 else 2048, 100)):
        rows = gen("dd", S, n, dtype, seed=n + S)
        views = as_columns(rows)
        assert views[0].stride() == (1, S)
        need = td.strided_large_workspace_bytes(n, S, S, 1, dtype, "cr")
        assert need > 0
        for algo, m in (("cr", 0), ("cr_pcr", 0), ("cr_pcr", 2), ("cr_pcr", 16), ("cr_pcr", 64),
                        ("cr_pcr", 256)):
            ref = td.solve_batched(*rows, algo=algo, switch_level=m)
            x = cols_solve(views, algo, m)
            assert x.stride() == (1, S)
            assert torch.equal(x.contiguous(), ref), (n, S, algo, m,
                                                      (x.contiguous() - ref).abs().max().item())
        e = err(*rows, x)
        assert e.max() <= TOL[dtype], (n, S, e.max())


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_column_passes_several_levels_and_bottom(dtype):
    """bottom_n below 32 R forces more passes; results stay bitwise."""
    chunk = td.column_chunk(dtype)
    n, S = (4096, 70) if dtype == torch.float32 else (2048, 70)
    rows = gen("dd", S, n, dtype, seed=7)
    views = as_columns(rows)
    ref = td.solve_batched(*rows, algo="cr")
    for bottom in (chunk // 2, chunk, 2 * chunk, 8 * chunk):
        x = cols_solve(views, "cr", bottom=bottom)
        assert torch.equal(x.contiguous(), ref), bottom
    ref = td.solve_batched(*rows, algo="cr_pcr", switch_level=32)
    x = cols_solve(views, "cr_pcr", 32, bottom=chunk)
    assert torch.equal(x.contiguous(), ref)


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_column_passes_ragged_n_and_in_place(dtype):
    for n, S in ((1000, 45), (3000, 32), (2049, 7)):
        if n > td.max_n(dtype, "cr"):
            continue
        rows = gen("dd", S, n, dtype, seed=n)
        views = as_columns(rows)
        ref = td.solve_batched(*rows, algo="cr_pcr")
        x = cols_solve(views, "cr_pcr")
        assert torch.equal(x.contiguous(), ref), n
        # guard: the grid's other elements are untouched by an in-place solve
        dcol = views[3]
        keep = views[0].clone()
        cols_solve(views[:3] + [dcol], "cr_pcr", x=dcol)
        assert torch.equal(dcol.contiguous(), ref), n
        assert torch.equal(views[0], keep)
        assert err(*rows, ref).max() <= TOL[dtype]


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_column_passes_cr_rd(dtype):
    n = 4096 if dtype == torch.float32 else 2048
    rows = gen("rdw", 50, n, dtype, seed=3)
    views = as_columns(rows)
    for m in (0, 8, 64, 256):
        ref = td.solve_batched(*rows, algo="cr_rd", switch_level=m)
        x = cols_solve(views, "cr_rd", m)
        # the RD inner's block scan association depends on how the m-system
        # is spread over lanes (R25), which differs between the
        # reduced interleaved system and the contiguous kernel: tolerance only
        assert err(*rows, x).max() <= TOL[dtype], m
        assert oracle.normwise_error(x.contiguous().cpu().numpy(),
                                     ref.cpu().numpy()).max() <= TOL[dtype], m


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_columns_beyond_max_n(dtype):
    """Column systems longer than tridiag_max_n (only the passes can hold
    them): bitwise equal to the row large-n path at the same m."""
    n, S = 1 << 15, 40
    rows = gen("dd", S, n, dtype, seed=11)
    views = as_columns(rows)
    for algo, m in (("cr", 0), ("cr_pcr", 32)):
        ref = td.solve_batched_large(*rows, algo=algo, switch_level=m)
        x = cols_solve(views, algo, m)
        assert torch.equal(x.contiguous(), ref), algo
        assert err(*rows, x).max() <= TOL[dtype], algo


def test_pcr_and_large_m_fall_back_to_on_chip_strided():
    """No CR levels to pass (PCR) or an m the passes cannot reach: the
    on-chip strided kernels, no workspace."""
    dtype = torch.float32
    n, S = 2048, 40
    rows = gen("dd", S, n, dtype, seed=5)
    views = as_columns(rows)
    assert td.strided_large_workspace_bytes(n, S, S, 1, dtype, "pcr") == 0
    assert td.strided_large_workspace_bytes(n, S, S, 1, dtype, "cr_pcr", 2048) == 0
    # m = 1024: one column pass of one CR level, PCR on the reduced rows
    assert td.strided_large_workspace_bytes(n, S, S, 1, dtype, "cr_pcr", 1024) > 0
    for algo, m in (("pcr", 0), ("cr_pcr", 2048), ("cr_pcr", 1024)):
        ref = td.solve_batched(*rows, algo=algo, switch_level=m)
        x = cols_solve(views, algo, m)
        assert torch.equal(x.contiguous(), ref), algo


def test_column_sweep_of_a_grid_full_size_sampled():
    """The bench workload (C3 column sweep, 4096 x 4096 fp32, CR+PCR at the
    tuned m): every system's relative residual, and 64 sampled systems vs
    fp64 Thomas."""
    n = S = 4096
    rows = gen("dd", S, n, torch.float32, seed=20100109 + 3)
    views = as_columns(rows)
    x = cols_solve(views, "cr_pcr").contiguous()
    a, b, c, d = [t.double() for t in rows]
    xd = x.double()
    ax = b * xd
    ax[:, 1:] += a[:, 1:] * xd[:, :-1]
    ax[:, :-1] += c[:, :-1] * xd[:, 1:]
    res = (ax - d).abs().amax(1) / d.abs().amax(1)
    assert torch.isfinite(res).all() and res.max().item() <= 1e-5, res.max().item()
    idx = torch.randperm(S, generator=torch.Generator().manual_seed(0))[:64].tolist()
    sub = [t[idx] for t in rows]
    assert err(*sub, x[idx]).max() <= TOL[torch.float32]




@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_single_system_view_with_both_strides_above_one(dtype):
    """one system whose element stride and system stride are
    both > 1 -- e.g. a column of a grid, ``grid[:, j].unsqueeze(0)`` (strides
    (N*N, N)) or ``t[0:1, ::2]`` -- is read and written through its element
    stride (bitwise equal to the contiguous solve) and nothing else in the
    parent buffer is touched, also in place (x == d)."""
    for n in (5, 64, 500, 512, 2048, 4096):
        if n > td.max_n(dtype, "cr"):
            continue
        N = n
        rows = gen("dd", 1, n, dtype, seed=n)
        for algo in ("cr", "cr_pcr", "pcr") if n <= td.max_n(dtype, "pcr") else ("cr", "cr_pcr"):
            ref = td.solve_batched(*rows, algo=algo)
            torch.cuda.synchronize()
            views, grids = [], []
            for t in rows:
                g = torch.full((N, N + 3), 9.0, dtype=dtype, device="cuda")
                g[:, 1] = t[0]
                grids.append(g)
                views.append(g[:, 1].unsqueeze(0))  # shape (1, n), element stride N + 3
            assert views[0].stride()[1] == N + 3 and views[0].stride()[0] > 1
            xg = torch.full((N, N + 3), 5.0, dtype=dtype, device="cuda")
            xv = xg[:, 1].unsqueeze(0)
            td.solve_batched(*views, x=xv, algo=algo)
            torch.cuda.synchronize()
            assert torch.equal(xv.contiguous(), ref), (n, algo)
            mask = torch.ones_like(xg, dtype=torch.bool)
            mask[:, 1] = False
            assert bool((xg[mask] == 5.0).all()), (n, algo)
            # in place through the same view
            dv = views[3]
            td.solve_batched(views[0], views[1], views[2], dv, x=dv, algo=algo)
            torch.cuda.synchronize()
            assert torch.equal(dv.contiguous(), ref), (n, algo)
            assert bool((grids[3][mask] == 9.0).all()), (n, algo)
        # every other element of a row: t[0:1, ::2]
        wide = [torch.stack([t[0], torch.full_like(t[0], 3.0)], dim=1).reshape(1, 2 * n) for t in rows]
        sv = [w[0:1, ::2] for w in wide]
        assert sv[0].stride() == (2 * n, 2)
        xw = torch.full((1, 2 * n), 4.0, dtype=dtype, device="cuda")
        td.solve_batched(*sv, x=xw[0:1, ::2], algo="cr")
        torch.cuda.synchronize()
        assert torch.equal(xw[0, ::2], td.solve_batched(*rows, algo="cr")[0]), n
        assert bool((xw[0, 1::2] == 4.0).all()), n


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_column_unit_order_is_bitwise_neutral(dtype, monkeypatch):
    """The row-aligned unit orders of the column passes (TRIDIAG_COL_ORDER=1,
    default: chunk-major expansion, grid = groups x pieces reduction) change
    only which CTA computes which unit: bitwise the same x as the group-major
    order, for full and ragged 32-system groups and several grid shapes."""
    for n, S in ((4096 if dtype == torch.float32 else 2048, 100), (1024, 33), (2048, 600)):
        rows = gen("dd", S, n, dtype, seed=n + S)
        views = as_columns(rows)
        out = {}
        for v in ("1", "0"):
            monkeypatch.setenv("TRIDIAG_COL_ORDER", v)
            td.reload_knobs()
            out[v] = cols_solve(views, "cr_pcr").contiguous()
        monkeypatch.delenv("TRIDIAG_COL_ORDER")
        td.reload_knobs()
        assert torch.equal(out["1"], out["0"]), (n, S)
        assert torch.equal(out["1"], td.solve_batched(*rows, algo="cr_pcr")), (n, S)
