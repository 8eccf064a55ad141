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
# CTA kernel (n > 32 R, tdg_cta_tma_kernel), warp 0 of every CTA
CTA_PHASES = ["wait for the TMA stage", "in-lane CR forward + next-warp heads (barrier 1)",
              "lane-level CR forward (barrier 2, lane-31 chain)",
              "survivor solve (barrier 3 .. barrier 4)", "lane-level back-substitution",
              "in-lane back-substitution", "store issue"]

CONFIGS = [("f32", 512, 131072, "cr_pcr", 32), ("f32", 512, 131072, "cr", 0),
           ("f32", 512, 131072, "cr_rd", 8), ("f32", 512, 131072, "cr_pcr", 128),
           ("f32", 512, 131072, "pcr", 0), ("f32", 512, 131072, "rd", 0),
           ("f32", 64, 1048576, "cr_pcr", 4), ("f64", 256, 262144, "cr_pcr", 32)]


def run_cta(dts, n, S, algo, m):
    dt = torch.float32 if dts == "f32" else torch.float64
    fam = "poi" if algo in ("rd", "cr_rd") else "dd"
    a, b, c, d = inputs.generate(fam, S, n, dt, device="cuda")
    for _ in range(3):
        td.solve_batched(a, b, c, d, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    st = td.phase_stamps().double()
    st = st[st[:, 0] > 0]
    out = {"dtype": dts, "n": n, "S": S, "algo": algo, "m": m, "kernel": "tdg_cta_tma_kernel",
           "samples": int(st.shape[0])}
    # systems after the first of each CTA (the first includes the launch ramp)
    first = st[0::4]
    steady = torch.cat([st[1::4], st[2::4], st[3::4]])
    for name, blk in (("first_system", first), ("steady", steady)):
        present = [j for j in range(8) if bool((blk[:, j] > 0).all())]
        ph = {}
        for j0, j1 in zip(present, present[1:]):
            ph[CTA_PHASES[j0] if j1 == j0 + 1 else f"{CTA_PHASES[j0]} .. {CTA_PHASES[j1 - 1]}"] = float((blk[:, j1] - blk[:, j0]).mean())
        tot = sum(ph.values())
        out[name] = {"cycles_per_system": tot,
                     "phases": {k: {"cycles": v, "share": v / tot} for k, v in ph.items()}}
    # wall between consecutive systems of a CTA (stage wait included)
    per = (st[1::4, 0] - st[0::4, 0])
    out["cycles_between_system_starts"] = float(per.mean())
    return out


PASS_PHASES = {
    "col_reduce": ["wait for the TMA stage", "in-lane CR forward", "heads barrier + tail chain",
                   "survivor stores"],
    "col_expand": ["x2 loads + wait for the TMA stage", "in-lane forward (recomputed)",
                   "in-lane back-substitution", "x stores"],
    "large_reduce": ["loads + KIN forward levels (lanes, warps, chunk heads)", "survivor stores"],
    "large_expand": ["loads + KIN forward levels (recomputed)", "in-lane back-substitution",
                     "x stores"],
}


def run_passes(dts, n, S, layout, algo="cr_pcr"):
    """Per-launch phase cycles of the multi-launch paths (column passes, large n)."""
    dt = torch.float32 if dts == "f32" else torch.float64
    g = inputs.generate("dd", S, n, dt, device="cuda")
    if layout == "cols":
        g = [t.t().contiguous().t() for t in g]
    for _ in range(2):
        td.solve_batched(*g, algo=algo)
    torch.cuda.synchronize()
    out = {"dtype": dts, "n": n, "S": S, "layout": layout, "algo": algo, "launches": []}
    for i, k in enumerate(td.last_kernel_names()):
        kind = next((key for key in PASS_PHASES if key in k), None)
        st = td.phase_stamps(launch=i).double()
        st = st[st[:, 0] > 0]
        rec = {"launch": i, "kernel": k[:60], "units": int(st.shape[0])}
        if kind is not None and st.shape[0] > 0:
            names = PASS_PHASES[kind]
            dl = (st[:, 1:len(names) + 1] - st[:, 0:len(names)]).mean(0).tolist()
            tot = sum(dl)
            rec["pass"] = kind
            rec["cycles_per_unit"] = tot
            rec["phases"] = {nm: {"cycles": v, "share": v / tot} for nm, v in zip(names, dl)}
        out["launches"].append(rec)
    return out


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


CTA_CONFIGS = [("f32", 4096, 4096, "cr_pcr", 0), ("f64", 4096, 4096, "cr_pcr", 0),
               ("f32", 8192, 16384, "cr_pcr", 0), ("f32", 2048, 32768, "cr_pcr", 0),
               ("f32", 4096, 4096, "rd", 0), ("f32", 4096, 4096, "cr", 0)]

if __name__ == "__main__":
    td.load(build_if_missing=False)
    which = sys.argv[1] if len(sys.argv) > 1 else "all"
    if which in ("all", "warp"):
        for cfg in CONFIGS:
            print(json.dumps(run(*cfg)), flush=True)
    if which in ("all", "cta"):
        for cfg in CTA_CONFIGS:
            print(json.dumps(run_cta(*cfg)), flush=True)
    if which in ("all", "passes"):
        for cfg in (("f32", 4096, 4096, "cols"), ("f64", 4096, 4096, "cols"),
                    ("f32", 1 << 20, 64, "rows"), ("f64", 1 << 20, 32, "rows")):
            print(json.dumps(run_passes(*cfg)), flush=True)
