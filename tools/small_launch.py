"""Per-launch time of small batches: rotating cold buffer sets vs one
L2-resident set, back-to-back launches (one event pair around K launches) vs
an event between launches.  Usage: small_launch.py > out.jsonl"""
import json
import math
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

K = 50
for n, S in ((128, 16384), (256, 16384), (512, 16384), (128, 65536), (512, 2048)):
    per = 5 * n * S * 4
    for mode in ("cold", "l2"):
        nsets = max(1, math.ceil(4 * 126 * 2**20 / per)) if mode == "cold" else 1
        sets = []
        for k in range(nsets):
            g = inputs.generate("dd", S, n, torch.float32, s0=k * S, device="cuda")
            sets.append((*g, torch.empty_like(g[3])))
        for i in range(5):
            td.solve_batched(*sets[i % nsets])
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for i in range(K):
            td.solve_batched(*sets[i % nsets])
        e1.record()
        torch.cuda.synchronize()
        b2b = e0.elapsed_time(e1) * 1e3 / K
        ev = [torch.cuda.Event(enable_timing=True) for _ in range(K + 1)]
        ev[0].record()
        for i in range(K):
            td.solve_batched(*sets[i % nsets])
            ev[i + 1].record()
        torch.cuda.synchronize()
        per_l = sorted(ev[i].elapsed_time(ev[i + 1]) * 1e3 for i in range(K))[K // 2]
        print(json.dumps({"n": n, "S": S, "mode": mode, "nsets": nsets, "mb": per / 2**20,
                          "us_b2b": round(b2b, 2), "us_evented": round(per_l, 2),
                          "ideal_us": round(per / 6.55e3 / 1e3 * 1e6 / 1e3, 2)}), flush=True)
        del sets
