"""Minimal driver for ncu captures: generate one batch on the GPU and launch
the solver `reps` times (the first launches are warm-up for -s)."""
import argparse
import os
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
p.add_argument("--family", default="dd")
p.add_argument("--reps", type=int, default=4)
p.add_argument("--layout", default="rows", choices=["rows", "cols", "ragged"])
a = p.parse_args()
dt = torch.float32 if a.dtype == "f32" else torch.float64
A, B, C, D = inputs.generate(a.family, a.systems, a.n, dt, device="cuda")
if a.layout == "cols":
    A, B, C, D = [t.t().contiguous().t() for t in (A, B, C, D)]
X = torch.empty_like(D)
torch.cuda.synchronize()
for _ in range(a.reps):
    if a.algo.startswith("paper_cr"):   # the paper's schedule (Fig 9 baseline), mode 0 / 1
        td.paper_cr(A, B, C, D, X, mode=1 if a.algo == "paper_cr1" else 0)
    else:
        td.solve_batched(A, B, C, D, X, algo=a.algo, switch_level=a.m)
torch.cuda.synchronize()
print("done", a)
