"""Per-phase cycles of the single-pass cluster column kernel (phase stamps,
TRIDIAG_PHASE_STAMPS=1): [0] group start, [1] stage arrived, [2] in-lane
forward + heads (cluster barrier 1), [3] tail chain + survivors sent (barrier
2), [4] reduced solve + x returned (barrier 3), [5] back-substituted + stored.
usage: TRIDIAG_PHASE_STAMPS=1 python tools/cluster_phases.py f32 4096 4096"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

dts, n, S = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
dt = torch.float32 if dts == "f32" else torch.float64
td.load(build_if_missing=False)
g = [t.t().contiguous().t() for t in inputs.generate("dd", S, n, dt, device="cuda")]
for _ in range(3):
    x = td.solve_batched(*g, algo="cr_pcr")
torch.cuda.synchronize()
names = td.last_kernel_names()
st = td.phase_stamps(launch=0, width=8).cpu().double()
st = st.reshape(-1, 4, 8)              # [cta][group][slot]
steady = st[:, 1:4, :6]
ok = (steady > 0).all(-1)
d = (steady[..., 1:] - steady[..., :-1])[ok]
tot = (steady[..., 5] - steady[..., 0])[ok]
names_ph = ["wait stage", "fwd+heads (b1)", "tail+send (b2)", "solve+x back (b3)", "bwd+store"]
out = {"kernel": names[0][:60], "dtype": dts, "n": n, "S": S, "groups_sampled": int(ok.sum()),
       "cycles_per_group": float(tot.mean()),
       "phases": {k: float(v) for k, v in zip(names_ph, d.mean(0).tolist())}}
print(json.dumps(out))
