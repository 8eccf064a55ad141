"""Fig 9 on B200: per-step times of the paper's
own CR schedule -- one CTA per system, n/2 threads, in place in shared
memory, a barrier per step (tridiag_paper_cr mode 0) -- against the paper's
stride-one timing control (mode 1, "bank-conflict-free ... an incorrect
algorithm, but is for timing comparison only"), plus whole-kernel
times of both and of the library's CR (register-blocked, no shared memory)
on the same batches.

Run with TRIDIAG_PHASE_STAMPS=1 (set here before the library loads).
Output: JSON lines; stamps are clock64() deltas of thread 0 of the first 512
CTAs (slot 0 start, 1 after load, 2..L after forward steps, then the 2x2
solve, the backward steps, the store).
"""
import json
import os
import sys

os.environ["TRIDIAG_PHASE_STAMPS"] = "1"
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402


def timed(fn, reps=20):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps * 1e3  # us


def stamps_of(fn, n):
    fn()
    torch.cuda.synchronize()
    st = td.phase_stamps().view(-1, 32).double()
    L = n.bit_length() - 1
    nslots = 1 + 1 + (L - 1) + 1 + (L - 1) + 1
    st = st[st[:, 0] > 0][:, :nslots]
    dl = (st[:, 1:] - st[:, :-1]).mean(0).tolist()
    names = (["load"] + [f"fwd{s + 1}" for s in range(L - 1)] + ["solve2x2"]
             + [f"bwd{s + 1}" for s in range(L - 1)] + ["store"])
    return {k: round(v, 1) for k, v in zip(names, dl)}, int(st.shape[0])


def main():
    td.load(build_if_missing=False)
    for dts, n, S in (("f32", 512, 512), ("f32", 512, 131072), ("f32", 256, 256), ("f64", 512, 512)):
        dt = torch.float32 if dts == "f32" else torch.float64
        a, b, c, d = inputs.generate("dd", S, n, dt, device="cuda")
        x = torch.empty_like(d)
        out = {"dtype": dts, "n": n, "S": S}
        for mode in (0, 1):
            steps, cnt = stamps_of(lambda: td.paper_cr(a, b, c, d, x, mode=mode), n)
            out[f"mode{mode}_cycles_per_step"] = steps
            out[f"mode{mode}_stamped_ctas"] = cnt
        os.environ["TRIDIAG_PHASE_STAMPS"] = "0"
        td.reload_knobs()
        out["us_paper_cr"] = timed(lambda: td.paper_cr(a, b, c, d, x, mode=0))
        out["us_paper_cr_stride_one"] = timed(lambda: td.paper_cr(a, b, c, d, x, mode=1))
        out["us_library_cr"] = timed(lambda: td.solve_batched(a, b, c, d, x, algo="cr"))
        out["us_library_cr_pcr"] = timed(lambda: td.solve_batched(a, b, c, d, x, algo="cr_pcr"))
        os.environ["TRIDIAG_PHASE_STAMPS"] = "1"
        td.reload_knobs()
        print(json.dumps(out), flush=True)


if __name__ == "__main__":
    main()
