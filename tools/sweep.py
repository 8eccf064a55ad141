"""Throughput / accuracy sweeps on one GPU.

  c5     hybrid switch-level sweep: S = 16384, n = 128..8192, fp32/fp64,
         CR+PCR and CR+RD at every valid m; throughput on DD (CR+RD on POI)
         plus max normwise error vs the oracle on DD and POI samples.
  c2     all five algorithms at n = 64..512 on HBM-scale batches (S*n = 2^26)
         and the literal paper shapes S = n (L2-resident; CUDA graph of 100
         launches over rotating buffer sets -> us per batch).
  c3     ADI-style 4096 x 4096, fp32 and fp64, all algorithms that fit.
  c4     2^20 x 256 fp32 on one GPU (the W = 1 point of the scaling row).
  large  n = 2^14 .. 2^24 beyond one CTA (NEXT f2), S*n = 2^26 (fp32) / 2^25
         (fp64), CR / CR+PCR / CR+RD through the reduction passes: algorithmic
         GB/s (5nT) and the pass model's traffic (each level read twice).

Writes one JSON object per point to stdout.  Timing: CUDA events on the
launching stream, warm-up first, working set >= 4x L2 via rotating buffer sets;
points whose launches take under 40 us are re-timed as a CUDA graph of the same
launches ("timing": "cuda_graph"), which removes the Python call's host time.
"""
import argparse
import json
import math
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle  # noqa: E402
import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

L2_BYTES = 126 * 1024 * 1024
PEAK = 6547.5
try:
    PEAK = float(json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                             "MEASURED_PEAKS.json")))["hbm_gbs"])
except Exception:
    pass


def make_sets(family, S, n, dt, min_bytes):
    T = 4 if dt == torch.float32 else 8
    per = 5 * S * n * T
    nsets = max(1, math.ceil(min_bytes / per))
    nsets = min(nsets, 64)
    sets = []
    for k in range(nsets):
        a, b, c, d = inputs.generate(family, S, n, dt, s0=k * S, device="cuda")
        sets.append((a, b, c, d, torch.empty_like(d)))
    return sets, per


LAST_TIMING = "events"


def time_point(sets, algo, m, steps=50, warmup=5):
    """Median / min seconds per launch.  CUDA events between back-to-back
    launches; a point whose launches are shorter than GRAPH_BELOW_S is
    re-timed as a CUDA graph of the same launches (rotating sets), so that it
    measures the kernels rather than the Python call's host time (~10 us).
    LAST_TIMING records which."""
    global LAST_TIMING
    st = torch.cuda.current_stream()
    for i in range(warmup):
        a, b, c, d, x = sets[i % len(sets)]
        td.solve_batched(a, b, c, d, x, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(steps + 1)]
    ev[0].record(st)
    for i in range(steps):
        a, b, c, d, x = sets[i % len(sets)]
        td.solve_batched(a, b, c, d, x, algo=algo, switch_level=m)
        ev[i + 1].record(st)
    torch.cuda.synchronize()
    per = [ev[i].elapsed_time(ev[i + 1]) * 1e-3 for i in range(steps)]
    LAST_TIMING = "events"
    if statistics.median(per) >= GRAPH_BELOW_S:
        return statistics.median(per), min(per)
    gs = torch.cuda.Stream()
    gs.wait_stream(st)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.stream(gs):
        td.solve_batched(*sets[0][:4], sets[0][4], algo=algo, switch_level=m)  # warm on this stream
        gs.synchronize()
        with torch.cuda.graph(g, stream=gs):
            for i in range(steps):
                a, b, c, d, x = sets[i % len(sets)]
                td.solve_batched(a, b, c, d, x, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    g.replay()
    torch.cuda.synchronize()
    reps = []
    for _ in range(5):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(st)
        g.replay()
        e1.record(st)
        torch.cuda.synchronize()
        reps.append(e0.elapsed_time(e1) * 1e-3 / steps)
    LAST_TIMING = "cuda_graph"
    return statistics.median(reps), min(reps)


GRAPH_BELOW_S = 40e-6


def accuracy(family, n, dt, algo, m, S=256, **kw):
    a, b, c, d = inputs.generate(family, S, n, dt, device="cuda", seed=4242, **kw)
    x = td.solve_batched(a, b, c, d, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    ha, hb, hc, hd = [t.cpu().numpy() for t in (a, b, c, d)]
    ref = oracle.thomas(ha, hb, hc, hd)
    e = oracle.normwise_error(x.cpu().numpy(), ref)
    fin = np.isfinite(e)
    res = oracle.residual_inf(ha, hb, hc, hd, x.cpu().numpy().astype(np.float64))
    return {"max_err": float(e[fin].max()) if fin.any() else None,
            "nonfinite": int((~fin).sum()), "systems": S,
            "max_residual": float(np.nanmax(res)) if fin.any() else None}


def emit(d):
    print(json.dumps(d), flush=True)


def c5(args):
    S = 16384
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        for n in [128, 256, 512, 1024, 2048, 4096, 8192]:
            for algo in ("cr_pcr", "cr_rd"):
                if n > td.max_n(dt, algo):
                    continue
                fam = "dd" if algo == "cr_pcr" else "poi"
                sets, per = make_sets(fam, S, n, dt, 4 * L2_BYTES)
                mx = td.max_switch_level(dt, algo, n)
                for lm in range(1, int(math.log2(n)) + 1):
                    m = 2 ** lm
                    if m > mx:
                        continue
                    med, mn = time_point(sets, algo, m, steps=args.steps)
                    row = {"config": "c5", "dtype": dts, "n": n, "S": S, "algo": algo, "m": m,
                           "time_family": fam, "timing": LAST_TIMING, "ms_median": med * 1e3, "ms_min": mn * 1e3,
                           "systems_per_s": S / med, "gbs": per / med / 1e9,
                           "frac_of_peak": per / med / 1e9 / PEAK,
                           "auto": m == td.auto_switch_level(n, dt, algo)}
                    if not args.no_acc:
                        row["acc_dd"] = accuracy("dd", n, dt, algo, m)
                        row["acc_poi"] = accuracy("poi", n, dt, algo, m)
                    emit(row)
                del sets
                torch.cuda.empty_cache()


def c2(args):
    dt = torch.float32
    for n in [64, 128, 256, 512]:
        S = (1 << 26) // n
        for algo in ("cr", "pcr", "rd", "cr_pcr", "cr_rd"):
            fam = "poi" if algo in ("rd", "cr_rd") else "dd"
            sets, per = make_sets(fam, S, n, dt, 0)
            ms = [0]
            if algo in td.HYBRIDS:
                ms = sorted({td.auto_switch_level(n, dt, algo), n // 2, 256 if algo == "cr_pcr" else 128} & set(
                    2 ** j for j in range(1, int(math.log2(n)) + 1)))
            for m in ms:
                med, mn = time_point(sets, algo, m, steps=args.steps)
                emit({"config": "c2-hbm", "dtype": "f32", "n": n, "S": S, "algo": algo, "m": m,
                      "time_family": fam, "ms_median": med * 1e3, "systems_per_s": S / med,
                      "gbs": per / med / 1e9, "frac_of_peak": per / med / 1e9 / PEAK})
            del sets
        torch.cuda.empty_cache()
    # literal paper shapes: S = n, L2 resident; graph of 100 launches on rotating sets
    for n in [64, 128, 256, 512]:
        S = n
        for algo in ("cr", "pcr", "rd", "cr_pcr", "cr_rd"):
            fam = "poi" if algo in ("rd", "cr_rd") else "dd"
            sets, per = make_sets(fam, S, n, dt, 4 * L2_BYTES)
            g = torch.cuda.CUDAGraph()
            st = torch.cuda.Stream()
            with torch.cuda.stream(st):
                for i in range(3):
                    a, b, c, d, x = sets[i % len(sets)]
                    td.solve_batched(a, b, c, d, x, algo=algo)
            torch.cuda.synchronize()
            with torch.cuda.graph(g, stream=st):
                for i in range(100):
                    a, b, c, d, x = sets[i % len(sets)]
                    td.solve_batched(a, b, c, d, x, algo=algo, stream=st)
            g.replay()
            torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for _ in range(5):
                g.replay()
            e1.record()
            torch.cuda.synchronize()
            us = e0.elapsed_time(e1) * 1e3 / 500
            emit({"config": "c2-literal", "dtype": "f32", "n": n, "S": S, "algo": algo,
                  "m": td.auto_switch_level(n, dt, algo) if algo in td.HYBRIDS else 0,
                  "us_per_batch": us, "systems_per_s": S / (us * 1e-6),
                  "paper_gtx280_ms": {"cr": 1.066, "pcr": 0.534, "rd": 0.612, "cr_pcr": 0.422,
                                      "cr_rd": 0.488}[algo] if n == 512 else None})
            del sets, g
        torch.cuda.empty_cache()


def c3(args):
    n, S = 4096, 4096
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        for algo in ("cr", "pcr", "rd", "cr_pcr", "cr_rd"):
            if n > td.max_n(dt, algo):
                continue
            fam = "poi" if algo in ("rd", "cr_rd") else "dd"
            sets, per = make_sets(fam, S, n, dt, 4 * L2_BYTES)
            med, mn = time_point(sets, algo, 0, steps=args.steps)
            row = {"config": "c3", "dtype": dts, "n": n, "S": S, "algo": algo,
                   "m": td.auto_switch_level(n, dt, algo) if algo in td.HYBRIDS else 0,
                   "time_family": fam, "ms_median": med * 1e3, "systems_per_s": S / med,
                   "gbs": per / med / 1e9, "frac_of_peak": per / med / 1e9 / PEAK}
            if not args.no_acc:
                row["acc"] = accuracy(fam, n, dt, algo, 0, S=64)
            emit(row)
            del sets
            torch.cuda.empty_cache()


def c4(args):
    n, S = 256, 1 << 20
    dt = torch.float32
    sets, per = make_sets("dd", S, n, dt, 0)
    for algo in ("cr", "cr_pcr"):
        med, mn = time_point(sets, algo, 0, steps=args.steps)
        emit({"config": "c4-w1", "dtype": "f32", "n": n, "S": S, "algo": algo,
              "m": td.auto_switch_level(n, dt, algo) if algo in td.HYBRIDS else 0,
              "ms_median": med * 1e3, "systems_per_s": S / med, "gbs": per / med / 1e9,
              "frac_of_peak": per / med / 1e9 / PEAK})


def large_traffic(n, T, LR, bottom):
    """HBM bytes per system of the large-n pipeline (tridiag_large.cuh):
    per level, reduce reads 4n writes 4n/R, expand reads 4n + n/R writes n
    (heads: 4 R T per chunk boundary); the bottom solve 5 n_last T."""
    tot = 0
    cur = n
    while cur > bottom:
        chunks = cur // (256 * (1 << LR))
        nxt = cur >> LR
        tot += (4 * cur + 4 * nxt) + (4 * cur + nxt + cur) + 4 * (1 << LR) * max(chunks - 1, 0)
        cur = nxt
    return (tot + 5 * cur) * T


def large(args):
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        T = 4 if dts == "f32" else 8
        LR = 4 if dts == "f32" else 3
        total = (1 << 26) if dts == "f32" else (1 << 25)
        for ln in range(14, 25):
            n = 1 << ln
            S = max(1, total // n)
            for algo in ("cr", "cr_pcr", "cr_rd"):
                fam = "rdw" if algo == "cr_rd" else "dd"
                sets, per = make_sets(fam, S, n, dt, 4 * L2_BYTES)
                med, mn = time_point(sets, algo, 0, steps=args.steps)
                model = large_traffic(n, T, LR, td.max_n(dt, "cr")) * S
                row = {"config": "large", "dtype": dts, "n": n, "S": S, "algo": algo,
                       "time_family": fam, "ms_median": med * 1e3, "ms_min": mn * 1e3,
                       "systems_per_s": S / med, "gbs": per / med / 1e9,
                       "frac_of_peak": per / med / 1e9 / PEAK,
                       "model_bytes_per_5nT": model / per,
                       "model_gbs": model / med / 1e9, "model_frac": model / med / 1e9 / PEAK}
                if not args.no_acc:
                    row["acc"] = accuracy(fam, n, dt, algo, 0, S=2)
                emit(row)
                del sets
                torch.cuda.empty_cache()


def adi(args):
    """ADI-style 2D sweeps on NY x NX row-major grids: the row sweep solves NY
    contiguous systems of n = NX, the column sweep NX interleaved systems of
    n = NY (element stride NX).  Both directions, CR+PCR, DD."""
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        T = 4 if dts == "f32" else 8
        for NY, NX in [(512, 8192), (8192, 512), (4096, 4096), (2048, 2048)]:
            if max(NY, NX) > td.max_n(dt, "cr_pcr"):
                continue
            nsets = max(1, math.ceil(4 * L2_BYTES / (5 * NY * NX * T)))
            sets = []
            for kk in range(nsets):
                g = inputs.generate("dd", NX, NY, dt, s0=kk * NX, device="cuda")  # columns as rows
                cols = [t.t().contiguous().t() for t in g]                          # (NX, NY) strides (1, NX)
                sets.append((*cols, torch.empty_like(cols[0])))
            per = 5 * NY * NX * T
            med, mn = time_point(sets, "cr_pcr", 0, steps=args.steps)
            emit({"config": "adi-column", "dtype": dts, "grid": [NY, NX], "n": NY, "S": NX,
                  "ms_median": med * 1e3, "gbs": per / med / 1e9, "frac_of_peak": per / med / 1e9 / PEAK})
            rows = [tuple(t.t() for t in st[:4]) + (st[4].t(),) for st in sets]   # (NY, NX) contiguous
            med, mn = time_point(rows, "cr_pcr", 0, steps=args.steps)
            emit({"config": "adi-row", "dtype": dts, "grid": [NY, NX], "n": NX, "S": NY,
                  "ms_median": med * 1e3, "gbs": per / med / 1e9, "frac_of_peak": per / med / 1e9 / PEAK})
            del sets, rows
            torch.cuda.empty_cache()


if __name__ == "__main__":
    p = argparse.ArgumentParser()
    p.add_argument("configs", nargs="+", choices=["c2", "c3", "c4", "c5", "adi", "large"])
    p.add_argument("--steps", type=int, default=30)
    p.add_argument("--no-acc", action="store_true")
    a = p.parse_args()
    td.load(build_if_missing=False)
    for cfg in a.configs:
        globals()[cfg](a)
