"""GPU parity of the large-n path (NEXT f2, n > tridiag_max_n):
reduction passes of log2 R CR levels, the on-chip solve of the reduced
system, expansion passes.

* bitwise: CR and CR+PCR through the passes equal the one-kernel path
  wherever both apply (bottom_n forces passes at on-chip sizes);
* G1/G2 tolerances against fp64 Thomas at n = 2^15 ... 2^20 (DD), CR+RD on
  the RD-stable rdw family, ragged n, in place x == d.
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


def err(a, b, c, d, x):
    h = [t.detach().cpu().numpy() for t in (a, b, c, d)]
    ref = oracle.thomas(*h)
    return oracle.normwise_error(x.detach().cpu().numpy(), ref)


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
@pytest.mark.parametrize("algo,m", [("cr", 0), ("cr_pcr", 2), ("cr_pcr", 16), ("cr_pcr", 32),
                                    ("cr_pcr", 256)])
def test_passes_are_bitwise_the_on_chip_path(dtype, algo, m):
    """(Explicit m: the auto m is resolved at the size the passes reduce to.)"""
    mx = td.max_n(dtype, "cr")
    chunk = td.large_chunk(dtype)
    for n in (mx // 2, mx):
        a, b, c, d = gen("dd", 37, n, dtype, seed=n)
        ref = td.solve_batched(a, b, c, d, algo=algo, switch_level=m)
        for bottom in (chunk // 2, chunk, mx // 2):
            if bottom >= n or (m and m > bottom):
                continue
            x = td.solve_batched_large(a, b, c, d, algo=algo, switch_level=m, bottom_n=bottom)
            torch.cuda.synchronize()
            assert torch.equal(x, ref), (algo, m, n, bottom, (x - ref).abs().max().item())


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_large_n_dd_against_thomas(dtype):
    for n, S in ((1 << 15, 5), (1 << 17, 3), (1 << 20, 2)):
        a, b, c, d = gen("dd", S, n, dtype, seed=n)
        for algo, m in (("cr", 0), ("cr_pcr", 0), ("cr_pcr", 256)):
            x = td.solve_batched(a, b, c, d, algo=algo, switch_level=m)  # routes to the large path
            e = err(a, b, c, d, x)
            assert e.max() <= TOL[dtype], (algo, m, n, e.max())


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_large_n_cr_rd_rdw(dtype):
    for n in (1 << 15, 1 << 18):
        a, b, c, d = gen("rdw", 3, n, dtype, seed=n)
        for m in (0, 64, 1024):
            x = td.solve_batched(a, b, c, d, algo="cr_rd", switch_level=m)
            e = err(a, b, c, d, x)
            assert e.max() <= TOL[dtype], (m, n, e.max())


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
def test_large_n_ragged_and_in_place(dtype):
    for n in (12289, 40000, 100003):
        a, b, c, d = gen("km", 3, n, dtype, seed=n)
        x = td.solve_batched(a, b, c, d, algo="cr_pcr")
        e = err(a, b, c, d, x)
        assert e.max() <= TOL[dtype], (n, e.max())
        d2 = d.clone()
        td.solve_batched(a, b, c, d2, x=d2, algo="cr_pcr")
        torch.cuda.synchronize()
        assert torch.equal(d2, x)
        # rdw through CR+RD (c_pad = 1 padding rows)
        a, b, c, d = gen("rdw", 2, n, dtype, seed=n)
        e = err(a, b, c, d, td.solve_batched(a, b, c, d, algo="cr_rd"))
        assert e.max() <= TOL[dtype], ("cr_rd", n, e.max())


def test_large_n_partition_invariant_and_launches():
    n = 1 << 16
    a, b, c, d = gen("dd", 6, n, torch.float32)
    x = td.solve_batched(a, b, c, d, algo="cr_pcr")
    parts = [td.solve_batched(a[i:i + 2], b[i:i + 2], c[i:i + 2], d[i:i + 2], algo="cr_pcr")
             for i in range(0, 6, 2)]
    torch.cuda.synchronize()
    assert torch.equal(torch.cat(parts), x)
    # 2^16 -> 2^12: reduce (the chunk heads carried inside it), one on-chip
    # launch, expand
    assert td.last_launch_count() == 3
    # the workspace is the caller's: an explicit one gives the same bits
    ws = torch.empty(td.large_workspace_bytes(n, 6, torch.float32, "cr_pcr"), dtype=torch.uint8,
                     device="cuda")
    y = td.solve_batched_large(a, b, c, d, algo="cr_pcr", workspace=ws)
    torch.cuda.synchronize()
    assert torch.equal(x, y)
    assert np.isfinite(y.cpu().numpy()).all()
