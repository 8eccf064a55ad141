"""The paper's literal batches (S = n, L2-resident) as CUDA graphs of 100
launches on rotating buffer sets: microseconds per batch, every algorithm."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

out = {}
for n in (64, 128, 256, 512):
    for dts in ("f32", "f64"):
        dt = torch.float32 if dts == "f32" else torch.float64
        sets = []
        for k in range(8):
            g = inputs.generate("dd" , n, n, dt, s0=k * n, device="cuda")
            sets.append((*g, torch.empty_like(g[3])))
        for algo in ("cr", "cr_pcr", "cr_rd"):
            st = torch.cuda.Stream()
            with torch.cuda.stream(st):
                for i in range(3):
                    td.solve_batched(*sets[i % 8][:4], x=sets[i % 8][4], algo=algo)
                st.synchronize()
                g = torch.cuda.CUDAGraph()
                with torch.cuda.graph(g, stream=st):
                    for i in range(100):
                        td.solve_batched(*sets[i % 8][:4], x=sets[i % 8][4], algo=algo)
            torch.cuda.synchronize()
            g.replay(); torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for _ in range(5):
                g.replay()
            e1.record()
            torch.cuda.synchronize()
            out[f"{dts}_n{n}_{algo}"] = round(e0.elapsed_time(e1) * 1e3 / 500, 2)
print(json.dumps({"us_per_batch": out, "small_cta": os.environ.get("TRIDIAG_SMALL_CTA", "1")}))
