import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, oracle
import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs
for dt in (torch.float64,):
    for n in (1024, 2048, 4096):
        a,b,c,d = inputs.generate("dd", 4, n, dt, device="cuda")
        ref = oracle.thomas(*[t.cpu().numpy() for t in (a,b,c,d)])
        for m in (2,4,8,16,32,64,128):
            x = td.solve_batched(a,b,c,d,algo="cr_pcr",switch_level=m).cpu().numpy()
            err = np.abs(x-ref)/np.abs(ref).max(axis=1,keepdims=True)
            bad = np.where(err[0] > 1e-12)[0]
            print(n, m, f"{err.max():.2e}", "bad idx (sys0):", bad[:20], len(bad))
