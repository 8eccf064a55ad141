"""Host-side cost per call (no synchronisation inside the loop): the Python
binding, the raw C-ABI call, and a torch op for scale.  One tiny batch, so
the GPU is never the bottleneck.  Usage: host_overhead.py"""
import json
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

N = 2000
res = {}
for n, S in ((64, 1), (512, 512)):
    a, b, c, d = inputs.generate("dd", S, n, torch.float32, device="cuda")
    x = torch.empty_like(d)
    st = torch.cuda.current_stream()
    for name, fn in (
            ("solve_batched", lambda: td.solve_batched(a, b, c, d, x=x)),
            ("solve_batched_alloc_x", lambda: td.solve_batched(a, b, c, d)),
            ("raw_c_abi", lambda: td.solve_batched_raw(a.data_ptr(), b.data_ptr(), c.data_ptr(),
                                                       d.data_ptr(), x.data_ptr(), n, S,
                                                       torch.float32, "cr_pcr", 0,
                                                       st.cuda_stream)),
            ("torch_add_", lambda: x.add_(1.0))):
        for _ in range(50):
            fn()
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        for _ in range(N):
            fn()
        t1 = time.perf_counter()
        torch.cuda.synchronize()
        res[f"{name}_n{n}_S{S}_us"] = round((t1 - t0) / N * 1e6, 2)
print(json.dumps(res))
