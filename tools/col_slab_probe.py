"""Probe: the ADI column sweep (4096 x 4096, interleaved) solved slab by slab
(consecutive column groups of `slab` systems, one strided-large call each) --
does the expansion pass re-read its slab from L2 when the slab fits?"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

td.load(build_if_missing=False)
flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
for dts in ("f32", "f64"):
    dt = torch.float32 if dts == "f32" else torch.float64
    T = 4 if dts == "f32" else 8
    n = S = 4096
    g = [t.t().contiguous().t() for t in inputs.generate("dd", S, n, dt, device="cuda")]
    x = torch.empty_like(g[3])
    ref = td.solve_batched(*g, algo="cr_pcr")
    for slab in (4096, 2048, 1024, 512, 256, 128):
        ws = torch.empty(td.strided_large_workspace_bytes(n, slab, S, 1, dt, "cr_pcr"), dtype=torch.uint8, device="cuda")
        def run():
            for s0 in range(0, S, slab):
                v = [t[s0:s0 + slab] for t in g]
                td.solve_batched_strided_large(*v, x=x[s0:s0 + slab], algo="cr_pcr", workspace=ws)
        run()
        torch.cuda.synchronize()
        assert torch.equal(x, ref)
        ts = []
        for _ in range(5):
            flush.zero_()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(); run(); e1.record()
            torch.cuda.synchronize()
            ts.append(e0.elapsed_time(e1) * 1e3)
        t = min(ts)
        print(json.dumps({"dtype": dts, "slab": slab, "us": t, "frac_5nT": 5 * n * S * T / (t * 1e-6) / 6535.4e9}), flush=True)
