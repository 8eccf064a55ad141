"""Per-phase time shares of the warp kernels (the B200 analogue of the
paper's Figs 8, 11, 13, 15, 16).

Runs each configuration with TRIDIAG_PHASE_STAMPS=1 (set below, before the
library loads), reads the clock64() stamps lane 0 of warp 0 of every CTA
recorded at the phase boundaries of its first 4 system groups, and prints the
mean cycles and share per phase.  The stamps are per-warp latencies: with 16
warps per SM interleaved, phase 1 (loads + in-lane forward) contains the HBM
latency the other warps hide."""
import json
import os
import sys

os.environ["TRIDIAG_PHASE_STAMPS"] = "1"
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

PHASES = ["loads + in-lane CR forward", "tail chain (next-lane heads)",
          "lane-level CR + inner PCR/RD", "in-lane back-substitution", "store issue"]

CONFIGS = [("f32", 512, 131072, "cr_pcr", 32), ("f32", 512, 131072, "cr", 0),
           ("f32", 512, 131072, "cr_rd", 8), ("f32", 512, 131072, "cr_pcr", 128),
           ("f32", 512, 131072, "pcr", 0), ("f32", 512, 131072, "rd", 0),
           ("f32", 64, 1048576, "cr_pcr", 4), ("f64", 256, 262144, "cr_pcr", 32)]


def run(dts, n, S, algo, m):
    dt = torch.float32 if dts == "f32" else torch.float64
    fam = "poi" if algo in ("rd", "cr_rd") else "dd"
    a, b, c, d = inputs.generate(fam, S, n, dt, device="cuda")
    for _ in range(3):
        x = td.solve_batched(a, b, c, d, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    st = td.phase_stamps().double()
    st = st[st[:, 0] > 0]
    deltas = st[:, 1:6] - st[:, 0:5]
    mean = deltas.mean(0)
    tot = float(mean.sum())
    return {"dtype": dts, "n": n, "S": S, "algo": algo, "m": m, "samples": int(st.shape[0]),
            "cycles_per_group": tot,
            "phases": {p: {"cycles": float(v), "share": float(v) / tot} for p, v in zip(PHASES, mean)}}


if __name__ == "__main__":
    td.load(build_if_missing=False)
    for cfg in CONFIGS:
        print(json.dumps(run(*cfg)), flush=True)
