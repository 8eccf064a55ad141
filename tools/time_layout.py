"""Time one solve configuration in a given memory layout (rows = contiguous,
cols = interleaved ADI column sweep, i.e. (S, n) views with strides (1, S)).
Usage: time_layout.py --n 512 --systems 131072 --layout cols [--algo cr_pcr]"""
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
p.add_argument("--n", type=int, default=512)
p.add_argument("--systems", type=int, default=131072)
p.add_argument("--dtype", default="f32")
p.add_argument("--algo", default="cr_pcr")
p.add_argument("--m", type=int, default=0)
p.add_argument("--layout", default="cols", choices=["rows", "cols"])
p.add_argument("--steps", type=int, default=20)
a = p.parse_args()
dt = torch.float32 if a.dtype == "f32" else torch.float64
T = 4 if a.dtype == "f32" else 8
per = 5 * a.n * a.systems * T
nsets = max(1, math.ceil(4 * 126 * 2**20 / per))
sets = []
for k in range(nsets):
    g = inputs.generate("dd", a.systems, a.n, dt, s0=k * a.systems, device="cuda")
    if a.layout == "cols":
        g = [t.t().contiguous().t() for t in g]
    sets.append((*g, torch.empty_like(g[3])))
for i in range(3):
    td.solve_batched(*sets[i % nsets], algo=a.algo, switch_level=a.m)
torch.cuda.synchronize()
ev = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps + 1)]
ev[0].record()
for i in range(a.steps):
    td.solve_batched(*sets[i % nsets], algo=a.algo, switch_level=a.m)
    ev[i + 1].record()
torch.cuda.synchronize()
t = statistics.median(ev[i].elapsed_time(ev[i + 1]) for i in range(a.steps)) / 1e3
peak = json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                   "MEASURED_PEAKS.json")))["hbm_gbs"]
print(json.dumps({"n": a.n, "S": a.systems, "dtype": a.dtype, "algo": a.algo, "m": a.m,
                  "layout": a.layout, "us": t * 1e6, "gbs": per / t / 1e9,
                  "frac": per / t / 1e9 / peak}))
