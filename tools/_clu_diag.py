import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs
dts, n, S = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
dt = torch.float32 if dts == "f32" else torch.float64
td.load(build_if_missing=False)
g = [t.t().contiguous().t() for t in inputs.generate("dd", S, n, dt, device="cuda")]
for _ in range(3):
    x = td.solve_batched(*g, algo="cr_pcr")
torch.cuda.synchronize()
st = td.phase_stamps(launch=0, width=8).cpu().double().reshape(-1, 4, 8)[:, 1:4, :]
ok = (st > 0).all(-1)
d = (st[..., 1:] - st[..., :-1])[ok].mean(0).tolist()
names = ["wait", "read+sync+issue", "interior fwd", "put heads", "sync1", "tail+send+sync2", "solve+sync3"]
print(json.dumps({"n": n, "dtype": dts, **{k: round(v) for k, v in zip(names, d)}}))
