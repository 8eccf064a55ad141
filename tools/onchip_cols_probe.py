"""Probe: the literal n x n column sweeps through the on-chip strided CTA kernel
(tridiag_solve_batched_strided, scalar strided loads) instead of the column
passes -- us per sweep in a CUDA graph, bitwise check against the passes."""
import json, os, sys
sys.path.insert(0, os.getcwd())
import torch
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs
td.load(build_if_missing=False)
out = {}
for dts, n in (("f64", 512), ("f32", 1024), ("f64", 1024), ("f32", 2048)):
    dt = torch.float32 if dts == "f32" else torch.float64
    sets = []
    for k in range(8):
        g = [t.t().contiguous().t() for t in inputs.generate("dd", n, n, dt, s0=k * n, device="cuda")]
        sets.append((*g, torch.empty_strided(g[3].shape, g[3].stride(), dtype=dt, device="cuda")))
    st = torch.cuda.Stream()
    def call(i):
        s = sets[i % 8]
        rc = td.solve_batched_strided_raw(*(t.data_ptr() for t in s), n, n, n, 1, dt, "cr_pcr", 0, st.cuda_stream)
        assert rc == 0, rc
    ref = td.solve_batched(*sets[0][:4], algo="cr_pcr")
    with torch.cuda.stream(st):
        call(0)
    torch.cuda.synchronize()
    eq = bool(torch.equal(sets[0][4], ref))
    with torch.cuda.stream(st):
        for i in range(3): call(i)
        st.synchronize()
        gr = torch.cuda.CUDAGraph()
        with torch.cuda.graph(gr, stream=st):
            for i in range(100): call(i)
    torch.cuda.synchronize(); gr.replay(); torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(5): gr.replay()
    e1.record(); torch.cuda.synchronize()
    out[f"{dts}_{n}x{n}_onchip_strided"] = {"us": round(e0.elapsed_time(e1) * 1e3 / 500, 2), "bitwise_eq_passes": eq, "kernels": [k[:40] for k in td.last_kernel_names()]}
print(json.dumps(out))
