"""Pitched-row timing (system stride > n): one point per (dtype, n, pitch)."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

for dts, n, extra in (("f32", 512, 16), ("f32", 500, 12), ("f32", 4096, 16), ("f64", 4096, 8)):
    dt = torch.float32 if dts == "f32" else torch.float64
    T = 4 if dts == "f32" else 8
    pitch = n + extra
    S = (1 << 26) // n if dts == "f32" else (1 << 25) // n
    rows = inputs.generate("dd", S, n, dt, device="cuda")
    bufs = [torch.empty((S, pitch), dtype=dt, device="cuda") for _ in range(5)]
    views = []
    for bf, t in zip(bufs, list(rows) + [rows[0]]):
        bf[:, :n] = t
        views.append(bf[:, :n])
    del rows
    for _ in range(3):
        td.solve_batched(*views[:4], x=views[4])
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(20):
        td.solve_batched(*views[:4], x=views[4])
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) / 20 * 1e-3
    gbs = 5 * n * T * S / t / 1e9
    print(json.dumps({"dtype": dts, "n": n, "pitch": pitch, "S": S, "us": round(t * 1e6, 1),
                      "gbs": round(gbs), "frac": round(gbs / 6547.5, 3),
                      "rag": os.environ.get("TRIDIAG_RAG_TMA", "1")}), flush=True)
    del bufs, views
    torch.cuda.empty_cache()
