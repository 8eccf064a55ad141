import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs
td.load(build_if_missing=False)
n, S = 1 << 20, 64
g = inputs.generate("dd", S, n, torch.float32, device="cuda")
x = torch.empty_like(g[3])
ref = td.solve_batched_large(*g, algo="cr_pcr")
flush = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
for slab in (64, 16, 8, 4, 2, 1):
    ws = torch.empty(td.large_workspace_bytes(n, slab, torch.float32, "cr_pcr"), dtype=torch.uint8, device="cuda")
    def run():
        for s0 in range(0, S, slab):
            td.solve_batched_large(*[t[s0:s0 + slab] for t in g], x=x[s0:s0 + slab], algo="cr_pcr", workspace=ws)
    run(); torch.cuda.synchronize()
    assert torch.equal(x, ref)
    ts = []
    for _ in range(3):
        flush.zero_()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(); run(); e1.record(); torch.cuda.synchronize()
        ts.append(e0.elapsed_time(e1) * 1e3)
    t = min(ts)
    print(json.dumps({"slab": slab, "us": t, "frac_5nT": 5 * n * S * 4 / (t * 1e-6) / 6535.4e9, "launches_per_call": td.last_launch_count()}), flush=True)
