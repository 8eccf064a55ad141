"""Phase stamps (the B200 analogue of the paper's
per-phase timing, Figs 8/11/13/15/16; and per step, Fig 9,
P:L905-925).

With TRIDIAG_PHASE_STAMPS=1 every kernel family records clock64() at its
phase boundaries (include/tridiag.h, tridiag_phase_stamps).  Checked here:
the stamps of each recorded unit are present and non-decreasing in phase
order (a phase can only start after the previous one ended on that warp);
the paper-schedule CR kernel records exactly one stamp per step, 2 log2 n - 1
steps plus load / store / start; the RD inner leaves the CR-only
phases empty; multi-launch calls keep every launch's stamps.
"""
import math

import pytest
import torch

import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module", autouse=True)
def _stamps_on():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    mp = pytest.MonkeyPatch()
    mp.setenv("TRIDIAG_PHASE_STAMPS", "1")
    td.load()
    td.reload_knobs()
    yield
    mp.undo()
    td.reload_knobs()


def gen(S, n, dtype=torch.float32, family="dd"):
    return inputs.generate(family, S, n, dtype, device="cuda")


def rows_of(st):
    """Rows that were recorded (a unit's slot 0 is set)."""
    return st[st[:, 0] > 0]


def check_monotone(st, slots):
    r = rows_of(st)
    assert r.shape[0] > 0
    sub = r[:, slots]
    assert bool((sub > 0).all()), sub[:4]
    assert bool((sub[:, 1:] >= sub[:, :-1]).all())
    return r


def test_warp_kernel_stamps():
    a, b, c, d = gen(131072, 512)
    td.solve_batched(a, b, c, d, algo="cr_pcr")
    torch.cuda.synchronize()
    check_monotone(td.phase_stamps(), [0, 1, 2, 3, 4, 5])


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_cta_kernel_stamps(dtype):
    a, b, c, d = gen(2048, 4096, dtype)
    td.solve_batched(a, b, c, d, algo="cr_pcr")
    torch.cuda.synchronize()
    assert any("tdg_cta_tma_kernel" in k for k in td.last_kernel_names())
    check_monotone(td.phase_stamps(), list(range(8)))
    # RD inner (CTA-blocked scan): no lane-level CR / survivor phases
    a, b, c, d = gen(2048, min(4096, td.max_n(dtype, "rd")), dtype, family="rdw")
    td.solve_batched(a, b, c, d, algo="rd")
    torch.cuda.synchronize()
    r = check_monotone(td.phase_stamps(), [0, 1, 2, 5, 6, 7])
    assert bool((r[:, 3] == 0).all() and (r[:, 4] == 0).all())


def test_column_pass_stamps_every_launch():
    n = S = 2048
    g = [t.t().contiguous().t() for t in gen(S, n)]
    td.solve_batched(*g, algo="cr_pcr")
    torch.cuda.synchronize()
    names = td.last_kernel_names()
    assert len(names) == 3 and "col_reduce" in names[0] and "col_expand" in names[2]
    check_monotone(td.phase_stamps(launch=0), [0, 1, 2, 3, 4])      # reduce
    check_monotone(td.phase_stamps(launch=2), [0, 1, 2, 3, 4])      # expand
    assert torch.equal(td.phase_stamps(launch=2), td.phase_stamps())  # last launch
    assert td.phase_stamps(launch=3).numel() == 0                   # no such launch


def test_large_pass_stamps():
    a, b, c, d = gen(8, 1 << 16)
    td.solve_batched(a, b, c, d, algo="cr_pcr")
    torch.cuda.synchronize()
    names = td.last_kernel_names()
    red = [i for i, k in enumerate(names) if "large_reduce" in k]
    exp = [i for i, k in enumerate(names) if "large_expand" in k]
    assert red and exp
    check_monotone(td.phase_stamps(launch=red[0]), [0, 1, 2])
    check_monotone(td.phase_stamps(launch=exp[-1]), [0, 1, 2, 3])


@pytest.mark.parametrize("n", [4, 64, 512])
def test_paper_schedule_one_stamp_per_step(n):
    """tridiag_paper_cr stamps start, load, each of the 2 log2 n - 1 CR steps
    (log2 n - 1 forward, the 2x2 solve, log2 n - 1 backward) and the
    store: 2 log2 n + 2 stamps per CTA, non-decreasing."""
    a, b, c, d = gen(600, n)
    td.paper_cr(a, b, c, d)
    torch.cuda.synchronize()
    st = td.phase_stamps(width=32)
    r = rows_of(st)
    assert r.shape[0] == 512                      # the first 512 CTAs are stamped
    L = int(math.log2(n))
    k = 2 * L + 2
    assert bool((r[:, :k] > 0).all()) and bool((r[:, k:] == 0).all())
    assert bool((r[:, 1:k] >= r[:, :k - 1]).all())
