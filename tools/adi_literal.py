"""The paper's ADI application at its literal grid sizes (n x n, fp32 / fp64,
L2-resident): one row sweep (contiguous systems) and one column sweep
(interleaved systems: element i of system s at s + i n) per ADI half-step,
each as CUDA graphs of 100 launches on rotating grids -- microseconds per
sweep, CR+PCR at the tuned m."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

td.load(build_if_missing=False)
out = {}
for n in (256, 512, 1024, 2048):
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        for layout in ("rows", "cols"):
            sets = []
            for k in range(8):
                g = inputs.generate("dd", n, n, dt, s0=k * n, device="cuda")
                if layout == "cols":
                    g = [t.t().contiguous().t() for t in g]
                x = torch.empty_strided(g[3].shape, g[3].stride(), dtype=dt, device="cuda")
                sets.append((*g, x))
            st = torch.cuda.Stream()
            ws = None
            if layout == "cols":
                need = td.strided_large_workspace_bytes(n, n, n, 1, dt, "cr_pcr")
                ws = torch.empty(max(need, 1), dtype=torch.uint8, device="cuda")

            def call(i):
                s = sets[i % 8]
                if layout == "cols":
                    td.solve_batched_strided_large(*s[:4], x=s[4], algo="cr_pcr", workspace=ws, stream=st)
                else:
                    td.solve_batched(*s[:4], x=s[4], algo="cr_pcr", stream=st)
            with torch.cuda.stream(st):
                for i in range(3):
                    call(i)
                st.synchronize()
                gr = torch.cuda.CUDAGraph()
                with torch.cuda.graph(gr, stream=st):
                    for i in range(100):
                        call(i)
            torch.cuda.synchronize()
            gr.replay()
            torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for _ in range(5):
                gr.replay()
            e1.record()
            torch.cuda.synchronize()
            us = e0.elapsed_time(e1) * 1e3 / 500
            out[f"{dts}_{n}x{n}_{layout}"] = {"us": round(us, 2),
                                              "kernels": [k[:40] for k in td.last_kernel_names()]}
print(json.dumps(out))
