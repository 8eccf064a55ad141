"""Metamorphic parity of the GPU kernels, independent of the oracle: scaling
equation i (a_i, b_i, c_i, d_i together) by 2^e_i is exact in floating point,
and every operation the kernels perform on an equation -- the correctly
rounded reciprocal of a pivot, k = a * (1/b), a - c k as a fused
multiply-add, the Cramer 2x2 solve, the RD matrix ratios -- carries that
factor through exactly (1/(2^e b) = 2^-e / b with correct rounding; an FMA of
exactly scaled operands is the scaled FMA).  So x must be BITWISE unchanged,
for every algorithm, kernel family and layout (a dropped or misplaced term
in any kernel would break the cancellation on some equation).  Exponents
within +-30 keep every intermediate far from overflow and subnormals.
"""
import pytest
import torch

import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    td.load()


def scaled(ts, seed):
    g = torch.Generator(device="cpu").manual_seed(seed)
    S, n = ts[0].shape
    e = torch.randint(-30, 31, (S, n), generator=g).to(torch.float64)
    f = torch.pow(2.0, e).to(device=ts[0].device, dtype=ts[0].dtype)
    return [t * f for t in ts]


CASES = [
    # (S, n, algo, m, family, layout)
    (300, 64, "cr", 0, "dd", "rows"),
    (300, 512, "cr_pcr", 0, "dd", "rows"),
    (300, 512, "cr_pcr", 256, "dd", "rows"),
    (300, 512, "pcr", 0, "dd", "rows"),
    (300, 256, "rd", 0, "rdw", "rows"),
    (300, 512, "cr_rd", 0, "rdw", "rows"),
    (40, 4096, "cr_pcr", 0, "dd", "rows"),
    (40, 4096, "rd", 0, "rdw", "rows"),
    (40, 1000, "cr_pcr", 0, "dd", "rows"),
    (301, 500, "cr_pcr", 0, "dd", "rows"),
    (3, 1 << 16, "cr_pcr", 0, "dd", "rows"),
    (64, 4096, "cr_pcr", 0, "dd", "cols"),
    (100, 512, "cr", 0, "dd", "cols"),
]


@pytest.mark.parametrize("dtype", [torch.float32, torch.float64], ids=["f32", "f64"])
@pytest.mark.parametrize("S,n,algo,m,family,layout", CASES)
def test_power_of_two_row_scaling_is_bitwise_invisible(dtype, S, n, algo, m, family, layout):
    if n > td.max_n_large(dtype, algo):
        pytest.skip("size beyond this algorithm's range")
    if algo in ("rd", "pcr") and n > td.max_n(dtype, algo):
        pytest.skip("size beyond this algorithm's on-chip range")
    rows = inputs.generate(family, S, n, dtype, seed=n + S, device="cuda")
    srows = scaled(rows, seed=S * 31 + n)
    if layout == "cols":
        rows = [t.t().contiguous().t() for t in rows]
        srows = [t.t().contiguous().t() for t in srows]
    x0 = td.solve_batched(*rows, algo=algo, switch_level=m)
    x1 = td.solve_batched(*srows, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    assert torch.isfinite(x0).all()
    assert torch.equal(x0, x1), (S, n, algo, m, family, layout, td.last_kernel_names())
