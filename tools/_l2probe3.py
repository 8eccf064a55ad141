import torch, json
flush = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
for mb in (8, 16, 32, 48, 64, 96):
    x = torch.ones(mb * (1 << 18), device="cuda")
    y = torch.empty(16, device="cuda")
    res = []
    for rep in range(5):
        flush.zero_()
        e = [torch.cuda.Event(enable_timing=True) for _ in range(4)]
        e[0].record(); torch.amax(x, 0, out=y[0]); e[1].record(); torch.amax(x, 0, out=y[1]); e[2].record(); torch.amax(x, 0, out=y[2]); e[3].record()
        torch.cuda.synchronize()
        res.append([e[i].elapsed_time(e[i + 1]) * 1e3 for i in range(3)])
    best = [min(r[i] for r in res) for i in range(3)]
    print(json.dumps({"MB": mb, "us_cold": best[0], "us_warm1": best[1], "us_warm2": best[2],
                      "GBs_cold": mb * 1.048576e6 / best[0] / 1e3, "GBs_warm": mb * 1.048576e6 / best[1] / 1e3}))
