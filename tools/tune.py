"""Time a list of (dtype, n, S, algo, m) points in ONE process (the library's
tuning knobs TRIDIAG_WARP_R / TRIDIAG_PREFETCH are read from the environment
once per process).  Prints one JSON line per point, tagged with the knobs."""
import argparse
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from sweep import L2_BYTES, PEAK, accuracy, make_sets, time_point  # noqa: E402

p = argparse.ArgumentParser()
p.add_argument("--dtype", default="f32")
p.add_argument("--ns", default="64,128,256,512")
p.add_argument("--elems", type=int, default=1 << 26, help="S*n per batch (0: use --systems)")
p.add_argument("--systems", type=int, default=16384)
p.add_argument("--algos", default="cr_pcr")
p.add_argument("--ms", default="0")
p.add_argument("--steps", type=int, default=30)
p.add_argument("--acc", action="store_true")
a = p.parse_args()
td.load(build_if_missing=False)
dt = torch.float32 if a.dtype == "f32" else torch.float64
knobs = {k: os.environ.get(k) for k in ("TRIDIAG_WARP_R", "TRIDIAG_PREFETCH")}
for n in map(int, a.ns.split(",")):
    S = a.elems // n if a.elems else a.systems
    for algo in a.algos.split(","):
        fam = "poi" if algo in ("rd", "cr_rd") else "dd"
        if n > td.max_n(dt, algo):
            continue
        sets, per = make_sets(fam, S, n, dt, 4 * L2_BYTES)
        for m in map(int, a.ms.split(",")):
            if m and (algo not in td.HYBRIDS or m > n):
                continue
            try:
                med, mn = time_point(sets, algo, m, steps=a.steps)
            except Exception as e:  # noqa: BLE001
                print(json.dumps({"n": n, "algo": algo, "m": m, "error": str(e), **knobs}), flush=True)
                continue
            row = {"dtype": a.dtype, "n": n, "S": S, "algo": algo, "m": m, **knobs,
                   "us": med * 1e6, "gbs": per / med / 1e9, "frac": per / med / 1e9 / PEAK}
            if a.acc:
                row["acc"] = accuracy(fam, n, dt, algo, m)
            print(json.dumps(row), flush=True)
        del sets
        torch.cuda.empty_cache()
