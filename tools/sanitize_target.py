"""Small launches of every kernel family, for compute-sanitizer
(racecheck / synccheck / memcheck / initcheck).  Checks results too."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle  # noqa: E402
import paper_conf_ppopp_zhangco10_b200 as td  # noqa: E402
from paper_conf_ppopp_zhangco10_b200 import inputs  # noqa: E402

CASES = [
    # (dtype, n, S, algo, m, layout)  -- one per kernel family
    (torch.float32, 512, 40, "cr_pcr", 0, "contig"),     # warp kernel, register path
    (torch.float32, 512, 40, "pcr", 0, "contig"),        # warp kernel, blocked inner
    (torch.float32, 64, 40, "cr_rd", 16, "contig"),      # blocked RD
    (torch.float32, 2048, 6, "cr_pcr", 0, "contig"),     # TMA CTA kernel
    (torch.float32, 2048, 6, "cr_pcr", 1024, "contig"),  # CTA kernel, shared-memory inner
    (torch.float64, 1024, 5, "cr_rd", 0, "contig"),      # TMA CTA kernel fp64
    (torch.float32, 100, 33, "cr_pcr", 0, "contig"),     # ragged n (general path)
    (torch.float32, 256, 30, "cr_pcr", 0, "column"),     # interleaved tile kernel
    (torch.float32, 1024, 12, "cr", 0, "column"),        # CTA general strided path
    (torch.float32, 2048, 6, "rd", 0, "contig"),         # TMA CTA kernel, CTA-blocked RD scan
    (torch.float64, 1024, 5, "cr_rd", 256, "contig"),    # same, k = 2 in-lane levels
    (torch.float32, 1000, 7, "rd", 0, "contig"),         # CTA-blocked RD, staged ragged path
    (torch.float32, 16384, 2, "cr_pcr", 0, "contig"),    # large-n passes
    (torch.float64, 12289, 2, "cr_rd", 0, "contig"),     # large-n passes, ragged, RD inner
    (torch.float32, 256, 40, "pcr", 0, "contig"),        # cyclic PCR relayout, 2 systems / warp
    (torch.float64, 256, 40, "pcr", 0, "contig"),        # same, fp64 slots
    (torch.float32, 2048, 64, "cr_pcr", 0, "column"),    # column passes, TMA-fed
    (torch.float32, 1000, 37, "cr_pcr", 0, "column"),    # column passes, direct loads, ragged
    (torch.float64, 2048, 40, "cr", 0, "column"),        # column passes fp64, two levels
    (torch.float32, 1000, 9, "cr_pcr", 0, "contig"),     # ragged rows: TMA CTA kernel, 3-D maps
    (torch.float64, 3000, 5, "cr_rd", 0, "contig"),      # same, fp64, RD inner
    (torch.float32, 500, 37, "cr_pcr", 0, "contig"),     # ragged rows: warp kernel, 16-byte lanes
    (torch.float64, 100, 41, "cr", 0, "contig"),         # same, fp64, 4 lanes per system
    (torch.float32, 1000, 9, "cr_pcr", 0, "pitched"),    # pitched ragged rows: TMA 3-D maps
    (torch.float32, 500, 37, "cr", 0, "pitched"),        # pitched ragged rows: warp 16-byte lanes
]

only = int(sys.argv[1]) if len(sys.argv) > 1 else None
bad = 0
for idx, (dt, n, S, algo, m, layout) in enumerate(CASES):
    if only is not None and idx != only:
        continue
    fam = "rdw" if algo in ("rd", "cr_rd") else "dd"
    a, b, c, d = inputs.generate(fam, S, n, dt, device="cuda")
    if layout == "column":
        views = [t.t().contiguous().t() for t in (a, b, c, d)]
    elif layout == "pitched":
        views = []
        for t in (a, b, c, d):
            bf = torch.zeros((S, n + 12), dtype=dt, device="cuda")
            bf[:, :n] = t
            views.append(bf[:, :n])
    else:
        views = [a, b, c, d]
    x = td.solve_batched(*views, algo=algo, switch_level=m)
    torch.cuda.synchronize()
    ref = oracle.thomas(*[t.cpu().numpy() for t in (a, b, c, d)])
    e = float(np.max(oracle.normwise_error(x.contiguous().cpu().numpy(), ref)))
    tol = 1e-4 if dt == torch.float32 else 1e-10
    ok = e <= tol
    bad += not ok
    print(f"case {idx}: {dt} n={n} S={S} {algo} m={m} {layout}: err {e:.2e} {'ok' if ok else 'FAIL'}")
sys.exit(1 if bad else 0)
