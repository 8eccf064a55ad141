"""Quick timing of a few points (iteration tool): python tools/quick_bench.py
"f32,512,131072,pcr,0" "f32,4096,4096,cr_pcr,0,cols" ...  Prints one JSON line
per point: device time per launch (CUDA events, rotating buffer sets >= 4x L2)
and the fraction of the measured HBM copy peak on the algorithmic 5nT bytes."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

PEAK = 6535.4
try:
    PEAK = float(json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                             "MEASURED_PEAKS.json")))["hbm_gbs"])
except Exception:
    pass


def point(spec, steps=30):
    f = spec.split(",")
    dts, n, S, algo, m = f[0], int(f[1]), int(f[2]), f[3], int(f[4])
    layout = f[5] if len(f) > 5 else "rows"
    dt = torch.float32 if dts == "f32" else torch.float64
    T = 4 if dts == "f32" else 8
    fam = "rdw" if algo in ("rd", "cr_rd") and n > 512 else ("poi" if algo in ("rd", "cr_rd") else "dd")
    per = 5 * n * S * T
    nsets = max(1, min(16, -(-4 * 126 * 2**20 // per)))
    sets = []
    for kk in range(nsets):
        g = inputs.generate(fam, S, n, dt, s0=kk * S, device="cuda")
        if layout == "cols":
            g = [t.t().contiguous().t() for t in g]
        sets.append((*g, torch.empty_like(g[3])))
    call = (lambda i: td.paper_cr(*sets[i % nsets], mode=m)) if algo == "paper_cr" else \
        (lambda i: td.solve_batched(*sets[i % nsets], algo=algo, switch_level=m))
    for i in range(3):
        call(i)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for i in range(steps):
        call(i)
    e1.record()
    torch.cuda.synchronize()
    t = e0.elapsed_time(e1) / steps * 1e-3
    return {"spec": spec, "us": t * 1e6, "frac": per / t / 1e9 / PEAK, "kernels": td.last_kernel_names()[:3]}


if __name__ == "__main__":
    td.load(build_if_missing=False)
    for spec in sys.argv[1:]:
        print(json.dumps(point(spec)), flush=True)
