"""Rows vs interleaved columns (the ADI row / column sweeps) over n, one
process: median of K launches per point, inputs rotated over > 4x L2.
Usage: layout_sweep.py [--elems 16777216] [--steps 20] > out.jsonl"""
import argparse
import json
import math
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

p = argparse.ArgumentParser()
p.add_argument("--elems", type=int, default=1 << 24, help="S * n per batch")
p.add_argument("--steps", type=int, default=20)
p.add_argument("--ns", default="64,128,256,512,1024,2048,4096")
p.add_argument("--dtypes", default="f32,f64")
p.add_argument("--algo", default="cr_pcr")
a = p.parse_args()
peak = json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                   "MEASURED_PEAKS.json")))["hbm_gbs"]
for dts in a.dtypes.split(","):
    dt = torch.float32 if dts == "f32" else torch.float64
    T = 4 if dts == "f32" else 8
    for n in [int(v) for v in a.ns.split(",")]:
        S = a.elems // n
        per = 5 * n * S * T
        nsets = max(1, math.ceil(4 * 126 * 2**20 / per))
        base = [inputs.generate("dd", S, n, dt, s0=k * S, device="cuda") for k in range(nsets)]
        for layout in ("rows", "cols"):
            sets = []
            for g in base:
                if layout == "cols":
                    g = [t.t().contiguous().t() for t in g]
                sets.append((*g, torch.empty_like(g[3])))
            for i in range(3):
                td.solve_batched(*sets[i % nsets], algo=a.algo)
            torch.cuda.synchronize()
            ev = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps + 1)]
            ev[0].record()
            for i in range(a.steps):
                td.solve_batched(*sets[i % nsets], algo=a.algo)
                ev[i + 1].record()
            torch.cuda.synchronize()
            t = statistics.median(ev[i].elapsed_time(ev[i + 1]) for i in range(a.steps)) / 1e3
            print(json.dumps({"dtype": dts, "n": n, "S": S, "algo": a.algo, "layout": layout,
                              "launches": td.last_launch_count(), "us": round(t * 1e6, 2),
                              "gbs": round(per / t / 1e9, 1), "frac": round(per / t / 1e9 / peak, 4)}),
                  flush=True)
            del sets
        del base
        torch.cuda.empty_cache()
