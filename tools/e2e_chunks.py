import sys, time, torch, os
sys.path.insert(0, os.getcwd())
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs
S, n = 131072, 512
a, b, c, d = [t.cpu().pin_memory() for t in inputs.generate("dd", S, n, torch.float32, device="cuda")]
x = torch.empty_like(d).pin_memory()
for chunk in (2048, 4096, 8192, 16384, 32768):
    ws = torch.empty(td.host_workspace_bytes(n, torch.float32, chunk), dtype=torch.uint8, device="cuda")
    td.solve_batched_host(a, b, c, d, x, chunk_systems=chunk, workspace=ws)
    t0 = time.perf_counter()
    for _ in range(5):
        td.solve_batched_host(a, b, c, d, x, chunk_systems=chunk, workspace=ws)
    el = (time.perf_counter() - t0) / 5
    print(chunk, f"{S / el:.3e} systems/s", f"H2D {4 * n * 4 * S / el / 1e9:.1f} GB/s")
    del ws
