#!/usr/bin/env python
"""Benchmark of the B200 batched tridiagonal solver (one JSON line on rank 0).

Metric (BASELINE.json): systems solved/s and achieved HBM GB/s (% of peak),
512x512 fp32.  A "step" is one pass of the whole hot path -- load, CR forward
reduction, intermediate handoff, inner PCR, CR back-substitution, store (all
SURVEY.md 8(a) rows of the best hybrid, CR+PCR at the tuned m) -- over one
batch of synthetic diagonally dominant input, i.e. ONE tridiag_solve_batched
launch.  The 512x512 paper batch is 5.2 MB (L2 resident, launch bound), so the
per-GPU workload is 256 such batches: S = 131072 systems of n = 512 (1.34 GB,
> 126 MB L2: no flush needed), the roofline row C2-HBM of SURVEY.md 8(d).

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl reference]
  torchrun --nproc-per-node N bench.py --gpus N ...   (weak scaling: S per GPU)

  python bench.py --gpus N ...   (no torchrun: spawns the N ranks itself)

--impl reference times the CPU oracle (multi-threaded fp64 Thomas, the
paper's MT solver) on this workload; there is no reference code to install.

After the timed loop the line certifies what was timed: the relative residual
of EVERY system, the count of systems with a non-finite x, and 256 sampled
systems per rank against the oracle (fp64 Thomas) -- "check" in the line.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

PEAK_FALLBACK_GBS = 6650.0
METRIC = "systems solved/s and achieved HBM GB/s (% of peak), 512x512 fp32, 1/2/4/8 B200"
UNIT = "systems/s"


def parse():
    p = argparse.ArgumentParser()
    p.add_argument("--gpus", type=int, default=1)
    p.add_argument("--steps", type=int, default=200)
    p.add_argument("--warmup", type=int, default=20)
    p.add_argument("--impl", default="b200", choices=["b200", "reference"])
    p.add_argument("--system-size", dest="n", type=int, default=512,
                   help="equations per system (named so torchrun does not claim it)")
    p.add_argument("--systems", type=int, default=131072, help="systems per GPU (weak scaling)")
    p.add_argument("--total-systems", type=int, default=0,
                   help="strong scaling: split this many systems over the ranks (C4: 1048576 x n=256)")
    p.add_argument("--dtype", default="f32", choices=["f32", "f64"])
    p.add_argument("--algo", default="cr_pcr")
    p.add_argument("--switch-level", type=int, default=0)
    p.add_argument("--family", default="dd")
    p.add_argument("--no-extras", action="store_true", help="skip per-algorithm table, e2e and cpu baseline")
    p.add_argument("--cpu-seconds", type=float, default=8.0, help="wall budget of the cpu_baseline leg")
    p.add_argument("--dump-x", default="", help="save each rank's x to <path>.rank<r>.pt (harness tests)")
    p.add_argument("--check-samples", type=int, default=256,
                   help="systems per rank compared with the oracle after the timed loop")
    p.add_argument("--dist-backend", default="nccl", choices=["nccl", "gloo"],
                   help="process group for the post-timing reductions (gloo: harness tests with "
                        "several ranks on one GPU)")
    return p.parse_args()


def measured_peak():
    path = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        with open(path) as f:
            j = json.load(f)
        return float(j["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs, copy best-of-10)"
    except Exception:
        return PEAK_FALLBACK_GBS, "fallback (B200_PROFILING.md)"


def ncu_traffic(kernel, n, dtype, S):
    """DRAM bytes per launch of `kernel` (mangled name, as launched) on this
    workload from the committed ncu --set full capture
    (profiles/ncu_traffic.json, keyed by kernel, then by workload)."""
    path = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    try:
        with open(path) as f:
            j = json.load(f)
        # ncu's mangled names may drop the last parameter codes: match by prefix
        for k, v in j.items():
            if kernel.startswith(k) or k.startswith(kernel):
                rec = v.get(f"{dtype}_n{n}_S{S}")
                if rec:
                    return rec
        return None
    except Exception:
        return None


def demangle(name):
    try:
        import subprocess
        r = subprocess.run(["c++filt"], input=name, capture_output=True, text=True, timeout=5)
        return r.stdout.strip() or name
    except Exception:
        return name


class ClockSampler:
    """Samples SM clock and throttle reasons with NVML every ~10 ms."""
    REASONS = {0x1: "gpu_idle", 0x2: "applications_clocks_setting", 0x4: "sw_power_cap",
               0x8: "hw_slowdown", 0x10: "sync_boost", 0x20: "sw_thermal_slowdown",
               0x40: "hw_thermal_slowdown", 0x80: "hw_power_brake_slowdown",
               0x100: "display_clock_setting"}

    def __init__(self, index):
        self.ok = False
        self.samples = []
        self.max_mhz = None
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            self.ok = True
        except Exception:
            pass
        self._stop = threading.Event()
        self._t = None

    def _run(self):
        while not self._stop.is_set():
            try:
                mhz = self.nv.nvmlDeviceGetClockInfo(self.h, self.nv.NVML_CLOCK_SM)
                rs = self.nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
                util = self.nv.nvmlDeviceGetUtilizationRates(self.h).gpu
                self.samples.append((mhz, rs, util))
            except Exception:
                pass
            time.sleep(0.01)

    def start(self):
        if self.ok:
            self._t = threading.Thread(target=self._run, daemon=True)
            self._t.start()

    def stop(self):
        if self._t:
            self._stop.set()
            self._t.join()

    def summary(self):
        if not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": self.max_mhz, "reasons": [], "samples": 0}
        loaded = [s for s in self.samples if s[2] > 0] or self.samples
        reasons = set()
        for _, rs, _ in loaded:
            for bit, name in self.REASONS.items():
                if rs & bit and name != "gpu_idle":
                    reasons.add(name)
        return {"sm_mhz": statistics.median(s[0] for s in loaded), "sm_max_mhz": self.max_mhz,
                "reasons": sorted(reasons), "samples": len(loaded)}


def cpu_cores():
    try:
        return len(os.sched_getaffinity(0))
    except Exception:
        return os.cpu_count() or 1


def cpu_model():
    try:
        with open("/proc/cpuinfo") as f:
            for line in f:
                if line.startswith("model name"):
                    return line.split(":", 1)[1].strip()
    except Exception:
        pass
    return "unknown"


CPU_CALL_SYSTEMS = 32768  # systems per oracle call, the same in cpu_baseline and --impl reference


def _cpu_sample(n, dtype_t, family):
    """The oracle's bounded sample of the workload: its first
    CPU_CALL_SYSTEMS systems, as the fp64 upcast (fp32 copy for the fp32 MT
    variant)."""
    import torch
    from paper_conf_ppopp_zhangco10_b200 import inputs
    return [t.to(torch.float64).numpy() for t in inputs.generate(family, CPU_CALL_SYSTEMS, n, dtype_t)]


def _time_oracle(arrs, threads, dtype, budget_s, max_reps=1000):
    import numpy as np
    import oracle
    a, b, c, d = arrs
    x = np.empty_like(d)
    oracle.thomas_mt(a, b, c, d, threads, dtype=dtype, out=x)  # warm
    reps, t0 = 0, time.perf_counter()
    while True:
        oracle.thomas_mt(a, b, c, d, threads, dtype=dtype, out=x)
        reps += 1
        el = time.perf_counter() - t0
        if el >= budget_s or reps >= max_reps:
            return reps, el


def cpu_baseline(n, S, dtype_t, family, budget_s):
    """The oracle (fp64 Thomas, multi-threaded like the paper's MT solver,
    P:L750-755) as it stands, on a bounded sample of the bench workload; plus
    the paper's other CPU columns (Fig 7): the MT solver in fp32
    (the paper's precision) and single-thread Thomas ("GE") in fp64 / fp32."""
    import numpy as np
    cores = cpu_cores()
    arrs = _cpu_sample(n, dtype_t, family)
    arrs32 = [np.ascontiguousarray(v, dtype=np.float32) for v in arrs]
    reps, el = _time_oracle(arrs, cores, np.float64, budget_s)
    v = reps * CPU_CALL_SYSTEMS / el
    variants = {}
    for name, ar, thr, dt in (("fp32_mt", arrs32, cores, np.float32),
                              ("fp64_1thread", arrs, 1, np.float64),
                              ("fp32_1thread", arrs32, 1, np.float32)):
        r2, e2 = _time_oracle(ar, thr, dt, max(0.5, budget_s / 4))
        sps = r2 * CPU_CALL_SYSTEMS / e2
        variants[name] = {"value": sps, "threads": thr, "reps": r2, "wall_s": round(e2, 3),
                          "gbs": sps * 5 * n * (4 if dt == np.float32 else 8) / 1e9}
    return {"value": v, "unit": UNIT, "cores": cores, "kind": "oracle",
            "sample": f"{reps} calls x {CPU_CALL_SYSTEMS} systems of n={n} ({family}, fp64 upcast of the "
                      f"{str(dtype_t).replace('torch.', '')} inputs) = {reps * CPU_CALL_SYSTEMS} of the "
                      f"workload's systems, fp64 Thomas on {cores} threads ({cpu_model()}), wall {el:.2f} s",
            "gbs": v * 5 * n * 8 / 1e9,
            "variants": variants}


def run_reference(args):
    """--impl reference: the CPU oracle timed as the reference arm, each step
    one oracle call on the same CPU_CALL_SYSTEMS-system sample as cpu_baseline
    (so the two timings of the same program agree)."""
    import numpy as np
    import oracle
    import torch
    from paper_conf_ppopp_zhangco10_b200.partition import dist_env

    rank, _, world = dist_env()
    if rank != 0:
        return 0
    dt = torch.float32 if args.dtype == "f32" else torch.float64
    n = args.n
    cores = cpu_cores()
    a, b, c, d = _cpu_sample(n, dt, args.family)
    x = np.empty_like(d)
    for _ in range(args.warmup):
        oracle.thomas_mt(a, b, c, d, cores, out=x)
    t0 = time.perf_counter()
    for _ in range(args.steps):
        oracle.thomas_mt(a, b, c, d, cores, out=x)
    el = time.perf_counter() - t0
    v = args.steps * CPU_CALL_SYSTEMS / el
    line = {
        "impl": "reference", "metric": METRIC, "value": v, "unit": UNIT, "n_gpus": args.gpus,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * el / args.steps,
        "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "f64",
        "data": "synthetic", "config": workload_config(args, 0),
        "cpu_baseline": {"value": v, "unit": UNIT, "cores": cores, "kind": "oracle",
                         "sample": f"each step: one call on {CPU_CALL_SYSTEMS} systems of n={n} "
                                   f"({args.family}) of the workload, fp64 Thomas (oracle) on {cores} "
                                   f"threads ({cpu_model()})"},
        "e2e": {"value": v, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


def spawn_ranks(args):
    """--gpus N without a torchrun environment: start the N ranks here (one
    process per GPU, the same environment torchrun would give them) and
    return the worst exit code.  Rank 0 prints the line."""
    import socket
    import subprocess
    sock = socket.socket()
    sock.bind(("127.0.0.1", 0))
    port = sock.getsockname()[1]
    sock.close()
    procs = []
    for r in range(args.gpus):
        env = dict(os.environ, RANK=str(r), LOCAL_RANK=str(r), WORLD_SIZE=str(args.gpus),
                   LOCAL_WORLD_SIZE=str(args.gpus), MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
        procs.append(subprocess.Popen([sys.executable, os.path.abspath(__file__), *sys.argv[1:]],
                                      env=env))
    rcs = [p.wait() for p in procs]
    return max(rcs, key=abs)


def workload_config(args, m):
    nbytes = 5 * args.n * (4 if args.dtype == "f32" else 8) * args.systems
    return {"workload": f"C2-HBM: {args.systems} systems x {args.n} equations {args.dtype} per GPU "
                        f"({args.systems * args.n // (512 * 512)} paper 512x512 batches), "
                        f"family {args.family}",
            "n": args.n, "num_systems_per_gpu": args.systems, "algo": args.algo,
            "switch_level": m, "family": args.family,
            "l2": f"inputs {nbytes / 1e9:.2f} GB per step > 126 MB L2 (no flush needed)",
            "parallelism": f"dp{args.gpus} (batch partition, no collective on the solve path)"}


def rank_workload(args, rank, world):
    """(first global system, systems on this rank, systems in the job, scaling).
    Weak scaling (default): every rank owns args.systems systems, rank r the
    global range [r*S, (r+1)*S).  Strong scaling (--total-systems T): the
    partitioner splits T contiguously (sizes differ by at most one)."""
    from paper_conf_ppopp_zhangco10_b200.partition import shard_range
    if args.total_systems:
        sh = shard_range(args.total_systems, world, rank)
        return sh.lo, sh.count, args.total_systems, "strong"
    return rank * args.systems, args.systems, world * args.systems, "weak"


def time_solves(td, bufs, n, S, algo, m, steps, warmup, stream):
    import torch
    a, b, c, d, x = bufs
    with torch.cuda.stream(stream):
        for _ in range(warmup):
            td.solve_batched(a, b, c, d, x, algo=algo, switch_level=m, stream=stream)
    torch.cuda.synchronize()
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(steps + 1)]
    launches = 0
    ev[0].record(stream)
    for i in range(steps):
        td.solve_batched(a, b, c, d, x, algo=algo, switch_level=m, stream=stream)
        launches += td.last_launch_count()
        ev[i + 1].record(stream)
    torch.cuda.synchronize()
    per = [ev[i].elapsed_time(ev[i + 1]) for i in range(steps)]
    return sum(per) / 1e3, per, launches


def verify(td, a, b, c, d, x, samples, s0):
    """Certify the timed result: relative residual ||Ax - d||_inf / ||d||_inf of
    EVERY system (fp64, on the device, in chunks), systems with a non-finite
    x, and `samples` seeded random systems against the oracle (fp64 Thomas on
    the exact upcast; normwise error, reading R18).  Max / sum over ranks."""
    import numpy as np
    import torch
    from paper_conf_ppopp_zhangco10_b200.partition import reduce_max, reduce_sum
    S = d.shape[0]
    res_max, nonfinite = 0.0, 0
    step = max(1, (1 << 24) // max(1, d.shape[1]))
    for lo in range(0, S, step):
        hi = min(S, lo + step)
        a64, b64, c64, d64, x64 = (t[lo:hi].double() for t in (a, b, c, d, x))
        r = b64 * x64 - d64
        r[:, 1:] += a64[:, 1:] * x64[:, :-1]
        r[:, :-1] += c64[:, :-1] * x64[:, 1:]
        rel = r.abs().amax(1) / d64.abs().amax(1).clamp_min(1e-300)
        bad = ~torch.isfinite(x64).all(1)
        nonfinite += int(bad.sum())
        rel = torch.where(bad, torch.full_like(rel, float("inf")), rel)
        res_max = max(res_max, float(rel.max()))
    err_max = 0.0
    k = min(samples, S)
    if k > 0:
        import oracle
        idx = torch.randperm(S, generator=torch.Generator().manual_seed(20100109 + s0))[:k]
        idx = idx.sort().values.to(d.device)
        ha, hb, hc, hd = (t.index_select(0, idx).double().cpu().numpy() for t in (a, b, c, d))
        ref = oracle.thomas(ha, hb, hc, hd)
        e = oracle.normwise_error(x.index_select(0, idx).cpu().numpy(), ref)
        err_max = float(np.max(e))
    return {"residual_max": reduce_max(res_max), "nonfinite": int(reduce_sum(nonfinite)),
            "error_max": reduce_max(err_max), "oracle_samples_per_rank": k,
            "how": "after the timed loop: relative residual of every system (fp64, device); "
                   f"{k} seeded random systems per rank vs the oracle (fp64 Thomas), normwise "
                   "max|x - x^|/max|x^| (R18); max / sum over ranks"}


def scatter_leg(td, args, world, rank, S, n, dt, T, m, reps=5, warmup=2):
    """scatter (root -> all) + solve + gather (all -> root) of a W * S batch
    that starts on rank 0; see partition.scatter_solve_gather."""
    import torch
    import torch.distributed as dist
    from paper_conf_ppopp_zhangco10_b200 import inputs
    from paper_conf_ppopp_zhangco10_b200.partition import reduce_max, scatter_solve_gather
    root = (None,) * 4
    if rank == 0:
        # the whole job's batch on rank 0, generated in 2^26-element pieces
        # (the generator's fp64 temporaries would need ~80 B per element at once)
        root = tuple(torch.empty((world * S, n), dtype=dt, device="cuda") for _ in range(4))
        step = max(1, (1 << 26) // n)
        for s0 in range(0, world * S, step):
            cnt = min(step, world * S - s0)
            for dst, src in zip(root, inputs.generate(args.family, cnt, n, dt, s0=s0, device="cuda")):
                dst[s0:s0 + cnt] = src

    def solve(a, b, c, d):
        return td.solve_batched(a, b, c, d, algo=args.algo, switch_level=m)

    ph = [0.0, 0.0, 0.0]
    tot = 0.0
    for it in range(warmup + reps):
        ev = [torch.cuda.Event(enable_timing=True) for _ in range(4)]
        dist.barrier()
        torch.cuda.synchronize()
        x_full, _ = scatter_solve_gather(root, (S, n), solve, events=ev)
        torch.cuda.synchronize()
        if it >= warmup:
            for i in range(3):
                ph[i] += ev[i].elapsed_time(ev[i + 1]) / 1e3
            tot += ev[0].elapsed_time(ev[3]) / 1e3
    t = reduce_max(tot / reps)
    phases = [reduce_max(v / reps) for v in ph]
    ok = None
    if rank == 0:
        # the gathered x is the whole batch's solve: the last shard (solved on
        # rank W-1) against rank 0 solving the same rows itself, bitwise
        lo = (world - 1) * S
        x_ref = td.solve_batched(*[r[lo:] for r in root], algo=args.algo, switch_level=m)
        ok = bool(torch.equal(x_full[lo:], x_ref))
    moved = 4 * (world - 1) * S * n * T + (world - 1) * S * n * T
    del root
    torch.cuda.empty_cache()
    return {"value": world * S / t, "unit": UNIT, "systems": world * S,
            "ms_per_step": 1e3 * t,
            "phase_ms_max_over_ranks": {"scatter": 1e3 * phases[0], "solve": 1e3 * phases[1],
                                        "gather": 1e3 * phases[2]},
            "bytes_over_links_per_step": moved,
            "link_gbs_root": moved / max(phases[0] + phases[2], 1e-12) / 1e9,
            "gathered_x_bitwise_equal_to_local_solve": ok,
            "how": "rank 0 holds all W*S systems; dist.scatter of a, b, c, d (NCCL over "
                   "NVLink/NVSwitch), solve per rank, dist.gather of x to rank 0; CUDA events "
                   f"per phase on each rank, {reps} reps after {warmup} warm-up, max over ranks. "
                   "Context for the paper's with-transfer column (P:L738-746), not the headline."}


def pcie_peaks(h, hx, reps=5):
    """Pinned host <-> device copy rates (GB/s, best of `reps`) of one
    buffer the size of d: the ceiling of the host-buffer path."""
    import torch
    dbuf = torch.empty(h.shape, dtype=h.dtype, device="cuda")
    nb = h.numel() * h.element_size()
    out = {}
    for name, fn in (("h2d_gbs", lambda: dbuf.copy_(h, non_blocking=True)),
                     ("d2h_gbs", lambda: hx.copy_(dbuf, non_blocking=True))):
        best = float("inf")
        for _ in range(reps):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            torch.cuda.synchronize()
            e0.record()
            fn()
            e1.record()
            torch.cuda.synchronize()
            best = min(best, e0.elapsed_time(e1) / 1e3)
        out[name] = nb / best / 1e9
    out["bytes"] = nb
    del dbuf
    return out


def main():
    args = parse()
    if args.impl == "reference":
        return run_reference(args)

    import torch
    import torch.distributed as dist

    import paper_conf_ppopp_zhangco10_b200 as td
    from paper_conf_ppopp_zhangco10_b200 import inputs
    from paper_conf_ppopp_zhangco10_b200.partition import dist_env, reduce_max

    rank, local, world = dist_env()
    if "WORLD_SIZE" not in os.environ and args.gpus > 1:
        return spawn_ranks(args)
    if world != args.gpus:
        print(f"bench.py: --gpus {args.gpus} but WORLD_SIZE={world}", file=sys.stderr)
        return 2
    ndev = torch.cuda.device_count()
    if args.dist_backend == "nccl" and world > ndev:
        print(f"bench.py: {world} NCCL ranks need {world} GPUs, {ndev} visible "
              f"(--dist-backend gloo runs several ranks on one GPU for harness tests)", file=sys.stderr)
        return 2
    dev = local if local < ndev else local % ndev  # (>1 rank per GPU only for harness tests)
    torch.cuda.set_device(dev)
    if world > 1:
        if args.dist_backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", dev))
        else:
            dist.init_process_group(args.dist_backend)
    td.load(build_if_missing=False)
    dt = torch.float32 if args.dtype == "f32" else torch.float64
    T = 4 if args.dtype == "f32" else 8
    n = args.n
    # Owner computes: this rank's systems are [s0, s0+S) of the global batch.
    s0, S, total, scaling = rank_workload(args, rank, world)
    args.systems = S
    m = args.switch_level or (td.auto_switch_level(n, dt, args.algo) if args.algo in td.HYBRIDS else 0)
    bytes_per_step = 5 * n * T * S
    a, b, c, d = inputs.generate(args.family, S, n, dt, s0=s0, device="cuda")
    x = torch.empty_like(d)
    stream = torch.cuda.Stream()
    sampler = ClockSampler(dev)

    # warm-up, then the timed region: barrier + sync on both sides, max over ranks
    with torch.cuda.stream(stream):
        for _ in range(args.warmup):
            td.solve_batched(a, b, c, d, x, algo=args.algo, switch_level=m, stream=stream)
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    sampler.start()
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps + 1)]
    launches = 0
    ev[0].record(stream)
    for i in range(args.steps):
        td.solve_batched(a, b, c, d, x, algo=args.algo, switch_level=m, stream=stream)
        launches += td.last_launch_count()
        ev[i + 1].record(stream)
    torch.cuda.synchronize()
    sampler.stop()
    per_launch_ms = [ev[i].elapsed_time(ev[i + 1]) for i in range(args.steps)]
    local_s = sum(per_launch_ms) / 1e3
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    t_max = reduce_max(local_s)
    value = total * args.steps / t_max
    ms_per_step = 1e3 * t_max / args.steps

    kernels = td.last_kernel_names()
    check = verify(td, a, b, c, d, x, args.check_samples, s0)
    if args.dump_x:
        torch.save({"s0": s0, "x": x.cpu()}, f"{args.dump_x}.rank{rank}.pt")

    peak, peak_src = measured_peak()
    kern_s = statistics.mean(per_launch_ms) / 1e3   # this rank's average launch duration
    achieved = bytes_per_step / kern_s / 1e9
    kname = kernels[0] if len(kernels) == 1 else None
    prof = ncu_traffic(kname, n, args.dtype, S) if kname else None
    roofline = {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                "frac": achieved / peak,
                "traffic": prof.get("dram_bytes_per_launch") if prof else None,
                "traffic_source": prof.get("source") if prof else "no ncu capture of this kernel on this workload",
                "algorithmic_bytes_per_launch": bytes_per_step,
                "peak_source": peak_src,
                "frac_of_8TBs": achieved / 8000.0,
                "kernel": demangle(kname) if kname else kernels,
                "kernel_mangled": kname}

    line = {"metric": METRIC, "value": value, "unit": UNIT, "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms_per_step,
            "higher_is_better": True, "scaling": scaling, "vs_baseline": None,
            "dtype": args.dtype, "data": "synthetic (counter-based seeded DD family, device-generated)",
            "config": workload_config(args, m), "roofline": roofline,
            "hbm_gbs_aggregate": value * 5 * n * T / 1e9,
            "systems_in_job": total,
            "gpu_launches": launches, "clocks": sampler.summary(),
            "check": check,
            # the error fields SURVEY.md 8(d) / 8(c) "Metrics" name, from the check
            "error": check["error_max"], "residual": check["residual_max"],
            "nonfinite": check["nonfinite"]}

    if not args.no_extras:
        # --- e2e: host (pinned) buffers through the C ABI, copies inside the timed region
        ha, hb, hc, hd = [t.cpu().pin_memory() for t in (a, b, c, d)]
        hx = torch.empty_like(hd).pin_memory()
        chunk = 16384
        ws = torch.empty(td.host_workspace_bytes(n, dt, chunk), dtype=torch.uint8, device="cuda")
        td.solve_batched_host(ha, hb, hc, hd, hx, algo=args.algo, switch_level=m,
                              chunk_systems=chunk, workspace=ws)
        e2e_steps = max(3, min(10, args.steps // 20))
        if world > 1:
            dist.barrier()
        t0 = time.perf_counter()
        for _ in range(e2e_steps):
            td.solve_batched_host(ha, hb, hc, hd, hx, algo=args.algo, switch_level=m,
                                  chunk_systems=chunk, workspace=ws)
        e2e_local = time.perf_counter() - t0
        e2e_t = reduce_max(e2e_local)
        pcie = pcie_peaks(hd, hx)
        h2d_b, d2h_b = 4 * n * T * S, n * T * S
        # full duplex: the pipeline cannot beat the slower of the two directions
        bound_s = max(h2d_b / (pcie["h2d_gbs"] * 1e9), d2h_b / (pcie["d2h_gbs"] * 1e9))
        line["e2e"] = {"value": total * e2e_steps / e2e_t, "unit": UNIT,
                       "h2d_bytes_per_step": h2d_b, "d2h_bytes_per_step": d2h_b,
                       "h2d_gbs": h2d_b * e2e_steps / e2e_t / 1e9,
                       "pcie_peaks": pcie,
                       "frac_of_copy_bound": bound_s / (e2e_t / e2e_steps),
                       "how": f"tridiag_solve_batched_host on pinned host buffers, {chunk}-system "
                              f"chunks pipelined over 3 streams, {e2e_steps} steps, wall clock "
                              f"around the blocking call, max over ranks; frac_of_copy_bound = "
                              f"max(H2D bytes / H2D peak, D2H bytes / D2H peak) / step time, "
                              f"peaks measured here with plain pinned cudaMemcpy"}
        del ws, ha, hb, hc, hd, hx
        # --- every algorithm on the same workload (RD family on the RD-stable POI input)
        per_algo = {}
        for algo in ("cr", "pcr", "rd", "cr_pcr", "cr_rd"):
            if n > td.max_n(dt, algo):
                continue
            fam = "poi" if algo in ("rd", "cr_rd") else args.family
            bufs = (a, b, c, d, x) if fam == args.family else (*inputs.generate(fam, S, n, dt, s0=s0, device="cuda"), x)
            ms = [0]
            if algo in td.HYBRIDS:
                ms = sorted({td.auto_switch_level(n, dt, algo), min(n, 256 if algo == "cr_pcr" else 128)})
            for mm in ms:
                steps = max(5, args.steps // 4)
                t, per, _ = time_solves(td, bufs, n, S, algo, mm, steps, 3, stream)
                tm = reduce_max(t)
                sps = total * steps / tm
                gbs = bytes_per_step / (t / steps) / 1e9
                key = algo if mm == 0 else f"{algo}_m{mm}"
                per_algo[key] = {"systems_per_s": sps, "gbs_per_gpu": gbs, "frac_of_peak": gbs / peak,
                                 "family": fam}
        line["per_algo"] = per_algo
        # the other BASELINE.json configs (CR+PCR at the tuned m, this rank's GPU):
        # C3 ADI-style 4096 x 4096 (row sweep contiguous, column sweep interleaved),
        # C4 2^20 x 256 on one GPU, C5's largest system n = 8192.
        del a, b, c, d, x
        torch.cuda.empty_cache()
        other = {}
        # plus RD at C3 (CTA-blocked scan; RD-stable rdw input) and the large-n
        # passes (NEXT f2) at S * n = 2^26.
        for name, dts, nn, SS, layout, oalgo, fam in (
                ("c3_f32_4096x4096_rows", "f32", 4096, 4096, "rows", "cr_pcr", "dd"),
                ("c3_f32_4096x4096_columns", "f32", 4096, 4096, "cols", "cr_pcr", "dd"),
                ("c3_f64_4096x4096_rows", "f64", 4096, 4096, "rows", "cr_pcr", "dd"),
                ("c3_f64_4096x4096_columns", "f64", 4096, 4096, "cols", "cr_pcr", "dd"),
                ("c3_f32_4096x4096_rows_rd", "f32", 4096, 4096, "rows", "rd", "rdw"),
                ("c4_f32_1048576x256", "f32", 256, 1 << 20, "rows", "cr_pcr", "dd"),
                ("c5_f32_16384x8192", "f32", 8192, 16384, "rows", "cr_pcr", "dd"),
                ("large_f32_64x1048576", "f32", 1 << 20, 64, "rows", "cr_pcr", "dd"),
                ("large_f64_32x1048576", "f64", 1 << 20, 32, "rows", "cr_pcr", "dd"),
                # ragged n (not a power of two; padded in-kernel, NEXT f2)
                ("ragged_f32_67108x1000", "f32", 1000, 67108, "rows", "cr_pcr", "dd"),
                ("ragged_f32_134217x500", "f32", 500, 134217, "rows", "cr_pcr", "dd")):
            dtt = torch.float32 if dts == "f32" else torch.float64
            TT = 4 if dts == "f32" else 8
            sets = []
            nsets = max(1, -(-4 * 126 * 2**20 // (5 * nn * SS * TT)))
            for kk in range(nsets):
                g = inputs.generate(fam, SS, nn, dtt, s0=kk * SS, device="cuda")
                if layout == "cols":
                    g = [t.t().contiguous().t() for t in g]
                sets.append((*g, torch.empty_like(g[3])))
            steps = max(5, args.steps // 10)
            for i in range(3):
                td.solve_batched(*sets[i % nsets], algo=oalgo, stream=stream)
            torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(stream)
            for i in range(steps):
                td.solve_batched(*sets[i % nsets], algo=oalgo, stream=stream)
            e1.record(stream)
            torch.cuda.synchronize()
            tt = reduce_max(e0.elapsed_time(e1) / 1e3 / steps)
            gbs = 5 * nn * TT * SS / tt / 1e9
            other[name] = {"systems_per_s_per_gpu": SS / tt, "gbs_per_gpu": gbs,
                           "frac_of_peak": gbs / peak, "layout": layout, "algo": oalgo,
                           "family": fam}
            del sets
            torch.cuda.empty_cache()
        line["other_configs"] = other
        if rank == 0:
            line["cpu_baseline"] = cpu_baseline(n, S, dt, args.family, args.cpu_seconds)
        line["paper_context"] = {"gtx280_cr_pcr_512x512_ms": 0.422,
                                 "gtx280_systems_per_s": 512 / 0.422e-3,
                                 "note": "PAPER.md Fig 15 (P:L1100); context only, not vs_baseline"}
        # --- NVLink "with transfer" context row (NEXT f4; the paper's PCIe
        # column, as a scatter from one GPU): rank 0 holds the whole
        # job's batch, scatters equal shards to every rank over NCCL, each rank
        # solves, x is gathered back to rank 0.  Device time (CUDA events on
        # each rank's stream), max over ranks.  Only with NCCL (one GPU per
        # rank); last, so that everything above is already in the line.
        if world > 1 and args.dist_backend == "nccl" and os.environ.get("TRIDIAG_BENCH_SCATTER", "1") != "0":
            try:
                line["scatter"] = scatter_leg(td, args, world, rank, S, n, dt, T, m)
            except Exception as e:  # context row only: keep the line
                line["scatter"] = {"error": f"{type(e).__name__}: {e}"}
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()
    if rank == 0:
        print(json.dumps(line), flush=True)
    return 0


if __name__ == "__main__":
    sys.exit(main())
