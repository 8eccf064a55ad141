"""Probe: does a pass that re-reads a slab right after another pass read it
hit L2?  Runs ONE solve of the ADI column sweep (mode col, 4096 x 4096
interleaved) or the large-n rows (mode large, 64 x 2^20 fp32) slab by slab,
for use under ncu --cache-control none (per-kernel dram bytes and L2 hit rate).

usage: python tools/l2_reuse_probe.py col|large SLAB [f32|f64]
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

mode, slab = sys.argv[1], int(sys.argv[2])
dt = torch.float64 if len(sys.argv) > 3 and sys.argv[3] == "f64" else torch.float32
td.load(build_if_missing=False)
if mode == "col":
    n = S = 4096
    g = [t.t().contiguous().t() for t in inputs.generate("dd", S, n, dt, device="cuda")]
    x = torch.empty_like(g[3])
    ws = torch.empty(td.strided_large_workspace_bytes(n, slab, S, 1, dt, "cr_pcr"), dtype=torch.uint8,
                     device="cuda")

    def run():
        for s0 in range(0, S, slab):
            td.solve_batched_strided_large(*[t[s0:s0 + slab] for t in g], x=x[s0:s0 + slab],
                                           algo="cr_pcr", workspace=ws)
else:
    n, S = 1 << 20, 64 if dt == torch.float32 else 32
    g = inputs.generate("dd", S, n, dt, device="cuda")
    x = torch.empty_like(g[3])
    ws = torch.empty(td.large_workspace_bytes(n, slab, dt, "cr_pcr"), dtype=torch.uint8, device="cuda")

    def run():
        for s0 in range(0, S, slab):
            td.solve_batched_large(*[t[s0:s0 + slab] for t in g], x=x[s0:s0 + slab], algo="cr_pcr",
                                   workspace=ws)
torch.cuda.synchronize()
run()
torch.cuda.synchronize()
print("done", mode, slab, td.last_launch_count(), td.last_kernel_names())
