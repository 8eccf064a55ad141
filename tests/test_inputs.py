"""The shared seeded input generator (no method arithmetic; CPU only)."""
import numpy as np
import pytest
import torch

from paper_conf_ppopp_zhangco10_b200 import inputs


def test_deterministic_and_shard_consistent():
    full = inputs.generate("dd", 12, 64, torch.float32, seed=9)
    again = inputs.generate("dd", 12, 64, torch.float32, seed=9)
    shard = inputs.generate("dd", 5, 64, torch.float32, seed=9, s0=7)
    for f, g, s in zip(full, again, shard):
        assert torch.equal(f, g)
        assert torch.equal(f[7:12], s)
    other = inputs.generate("dd", 12, 64, torch.float32, seed=10)
    assert not torch.equal(full[3], other[3])


def test_families_have_their_structure():
    n = 128
    a, b, c, d = [t.numpy() for t in inputs.generate("dd", 50, n, torch.float64)]
    a0, c0 = a.copy(), c.copy()
    a0[:, 0] = 0
    c0[:, -1] = 0
    assert np.all(np.abs(b) >= np.abs(a0) + np.abs(c0) + 1.0)   # strict dominance, margin >= 1
    assert np.all(np.abs(a) < 1) and np.all(np.abs(d) < 1)
    assert 0.3 < np.mean(b > 0) < 0.7                          # random sign
    a, b, c, d = [t.numpy() for t in inputs.generate("km", 10, n, torch.float64, E=100.0)]
    assert np.all(a < 0) and np.all(c < 0)
    assert np.allclose(b, 1 - a - c)
    assert np.array_equal(c[:, :-1], a[:, 1:])                   # symmetric
    a, b, c, d = [t.numpy() for t in inputs.generate("poi1", 3, n, torch.float64)]
    assert np.all(a == -1) and np.all(b == 2) and np.all(c == -1) and np.all(d == 1)
    a, b, c, d = [t.numpy() for t in inputs.generate("cv", 3, n, torch.float64)]
    for v in (a, b, c):
        assert np.all((v >= 0.9) & (v < 1.1))
    a, b, c, d = [t.numpy() for t in inputs.generate("rdw", 3, n, torch.float64)]
    assert np.all(np.abs(a) <= 0.01)
    for v in (b, c):
        assert np.all((v >= 0.99) & (v < 1.01))


def test_rdw_is_rd_stable_in_the_oracle():
    """The rdw family's premise: the oracle's RD (fp64 and fp32) stays close
    to Thomas at n = 4096, where RD on DD / KM overflows in fp32."""
    import oracle
    a, b, c, d = [t.numpy() for t in inputs.generate("rdw", 4, 4096, torch.float64)]
    ref = oracle.thomas(a, b, c, d)
    x64, _, _ = oracle.rd(a, b, c, d)
    assert oracle.normwise_error(x64, ref).max() < 1e-11
    a, b, c, d = [t.numpy() for t in inputs.generate("rdw", 4, 4096, torch.float32)]
    ref = oracle.thomas(a, b, c, d)
    x32, _, _ = oracle.rd(a, b, c, d, dtype=np.float32)
    assert np.isfinite(x32).all()
    assert oracle.normwise_error(x32, ref).max() < 1e-4


def test_poison_corners_and_rounding():
    a, b, c, d = inputs.generate("dd", 4, 16, torch.float32, poison_corners=True)
    assert torch.isnan(a[:, 0]).all() and torch.isnan(c[:, -1]).all()
    assert not torch.isnan(a[:, 1:]).any() and not torch.isnan(c[:, :-1]).any()
    a64 = inputs.generate("dd", 4, 16, torch.float64)[1]
    assert torch.equal(a64.to(torch.float32), b)


def test_uniform_has_24_bits_in_unit_interval():
    g = torch.arange(1 << 16, dtype=torch.int64)
    u = inputs.uniform(g, 1, 0)
    assert float(u.min()) >= 0.0 and float(u.max()) < 1.0
    assert torch.all(u * (1 << 24) == torch.floor(u * (1 << 24)))
    assert abs(float(u.mean()) - 0.5) < 0.01


@pytest.mark.parametrize("family", ["dd", "poi", "poi1", "rdw", "cv"])
def test_equation_ranges_are_the_columns_of_the_full_systems(family):
    """generate(..., i0, count) gives exactly columns [i0, i0+count) of the full
    (S, n) systems (how a 2^30-equation system is generated in pieces)."""
    S, n = 3, 100
    full = inputs.generate(family, S, n, torch.float64, s0=7)
    for cuts in ((0, 100), (0, 1, 100), (0, 37, 64, 99, 100)):
        parts = [inputs.generate(family, S, n, torch.float64, s0=7, i0=lo, count=hi - lo)
                 for lo, hi in zip(cuts, cuts[1:])]
        for k in range(4):
            assert torch.equal(torch.cat([p[k] for p in parts], dim=1), full[k]), (family, cuts, k)


def test_equation_ranges_rejected_where_unsupported():
    with pytest.raises(ValueError):
        inputs.generate("km", 2, 10, i0=2, count=3)
    with pytest.raises(ValueError):
        inputs.generate("dd", 2, 10, i0=8, count=3)
    with pytest.raises(ValueError):
        inputs.generate("dd", 2, 10, i0=1, count=3, poison_corners=True)
