import torch, json
flush = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
for mb in (8, 16, 32, 48, 64, 96, 128):
    x = torch.ones(mb * (1 << 20) // 4, device="cuda")
    out = []
    for rep in range(3):
        flush.zero_()
        e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
        e[0].record(); s1 = x.sum(); e[1].record(); s2 = x.sum(); e[2].record()
        torch.cuda.synchronize()
        out.append((e[0].elapsed_time(e[1]) * 1e3, e[1].elapsed_time(e[2]) * 1e3))
    t1 = min(o[0] for o in out); t2 = min(o[1] for o in out)
    print(json.dumps({"MB": mb, "first_us": t1, "second_us": t2, "first_GBs": mb * 1.048576e6 / t1 / 1e3, "second_GBs": mb * 1.048576e6 / t2 / 1e3}))
