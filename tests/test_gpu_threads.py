"""The C ABI is thread-safe and stream-ordered (SURVEY.md 8(b) "Execution"):
host threads solving different batches concurrently, each on its own CUDA
stream, get bitwise the results of the same solves run one after another, and
each thread's launch count / kernel log describes its own last call
(thread-local).  ctypes releases the GIL around every library call, so the
calls really overlap on the host; the four workloads take four different
kernel families (warp kernel, TMA CTA kernel, column passes, large-n passes).
"""
import threading

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


def _workloads():
    out = []
    for k, (S, n, layout, dtype) in enumerate([(4096, 512, "rows", torch.float32),
                                               (512, 4096, "rows", torch.float32),
                                               (256, 2048, "cols", torch.float64),
                                               (4, 1 << 16, "rows", torch.float32)]):
        g = inputs.generate("dd", S, n, dtype, seed=100 + k, device="cuda")
        if layout == "cols":
            g = [t.t().contiguous().t() for t in g]
        out.append(g)
    return out


def test_concurrent_threads_match_sequential():
    work = _workloads()
    ref = []
    counts = []
    for g in work:
        ref.append(td.solve_batched(*g, algo="cr_pcr"))
        torch.cuda.synchronize()
        counts.append(td.last_launch_count())
    results = [[] for _ in work]
    seen = [[] for _ in work]
    errors = []
    barrier = threading.Barrier(len(work))

    def worker(i):
        try:
            s = torch.cuda.Stream()
            barrier.wait()
            for _ in range(12):
                with torch.cuda.stream(s):
                    x = td.solve_batched(*work[i], algo="cr_pcr", stream=s)
                seen[i].append(td.last_launch_count())
                results[i].append((x, s))
            s.synchronize()
        except Exception as e:  # pragma: no cover - reported below
            errors.append(repr(e))

    threads = [threading.Thread(target=worker, args=(i,)) for i in range(len(work))]
    for t in threads:
        t.start()
    for t in threads:
        t.join(timeout=300)
    assert not errors, errors
    torch.cuda.synchronize()
    for i in range(len(work)):
        assert len(results[i]) == 12
        for x, _ in results[i]:
            assert torch.equal(x, ref[i]), i
        assert seen[i] == [counts[i]] * 12, (i, seen[i], counts[i])
