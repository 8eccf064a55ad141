"""Summaries of ncu --set full captures exported as CSV on the GPU box
(`ncu -i REP --page raw --csv` and the same with --print-kernel-base mangled),
so the large .ncu-rep files never travel back.

  python tools/ncu_csv_summary.py DIR NAME[:workload_key] ... [--md OUT.md] [--traffic OUT.json]

For every NAME, DIR/NAME.raw.csv (and DIR/NAME.mangled.csv for the mangled
kernel names) are read; each captured launch gets a markdown table of the key
metrics and the top warp stall reasons.  --traffic merges
`{mangled kernel: {workload_key: {dram_bytes_per_launch, ...}}}` into the
JSON file bench.py reads for roofline.traffic.
"""
import csv
import json
import os
import sys

KEYS = [
    ("launch__grid_size", "grid"), ("launch__block_size", "block"),
    ("launch__registers_per_thread", "registers/thread"),
    ("launch__shared_mem_per_block_dynamic", "dynamic smem/block"),
    ("launch__occupancy_limit_registers", "occupancy limit (registers)"),
    ("gpu__time_duration.sum", "duration"),
    ("dram__bytes_read.sum", "DRAM read"), ("dram__bytes_write.sum", "DRAM write"),
    ("dram__throughput.avg.pct_of_peak_sustained_elapsed", "DRAM throughput % of peak"),
    ("sm__throughput.avg.pct_of_peak_sustained_elapsed", "SM throughput %"),
    ("smsp__issue_active.avg.pct_of_peak_sustained_active", "issue active %"),
    ("sm__warps_active.avg.pct_of_peak_sustained_active", "achieved occupancy %"),
    ("smsp__inst_executed.sum", "warp instructions"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", "smem bank conflicts (ld)"),
    ("l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum", "smem bank conflicts (st)"),
    ("l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum", "smem ld wavefronts"),
    ("l1tex__data_pipe_lsu_wavefronts_mem_shared_op_st.sum", "smem st wavefronts"),
    ("smsp__sass_inst_executed_op_shared_ld.sum", "smem ld instructions"),
    ("smsp__sass_inst_executed_op_shared_st.sum", "smem st instructions"),
    ("lts__t_bytes.sum", "L2 bytes"),
    ("sm__cycles_elapsed.avg.per_second", "SM clock"),
]


def read(path):
    rows = list(csv.reader(open(path)))
    h, u = rows[0], rows[1]
    return h, u, rows[2:]


def num(v):
    try:
        return float(v.replace(",", ""))
    except ValueError:
        return None


def to_bytes(v, unit):
    x = num(v)
    if x is None:
        return None
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "KB": 1e3, "MB": 1e6, "GB": 1e9}
    return x * scale.get(unit, 1)


def main():
    args = sys.argv[1:]
    md_out = traffic_out = None
    if "--md" in args:
        i = args.index("--md"); md_out = args[i + 1]; del args[i:i + 2]
    if "--traffic" in args:
        i = args.index("--traffic"); traffic_out = args[i + 1]; del args[i:i + 2]
    d = args[0]
    md = []
    traffic = {}
    if traffic_out and os.path.exists(traffic_out):
        traffic = json.load(open(traffic_out))
    for spec in args[1:]:
        name, _, wkey = spec.partition(":")
        h, u, rows = read(os.path.join(d, f"{name}.raw.csv"))
        mpath = os.path.join(d, f"{name}.mangled.csv")
        mangled = []
        if os.path.exists(mpath):
            rows_m = list(csv.reader(open(mpath)))
            ki = rows_m[0].index("Kernel Name")
            mangled = [r[ki] for r in rows_m[1:] if len(r) > ki and r[ki].startswith("_Z")]
        for j, r in enumerate(rows):
            kn = r[h.index("Kernel Name")]
            km = mangled[j] if j < len(mangled) else None
            md += [f"### {name} launch {j}: `{kn[:160]}`", ""]
            if km:
                md += [f"mangled: `{km}`", ""]
            md += ["| metric | value | unit |", "|---|---|---|"]
            for k, label in KEYS:
                if k in h:
                    i = h.index(k)
                    md.append(f"| {label} (`{k}`) | {r[i]} | {u[i]} |")
            stalls = []
            for i, k in enumerate(h):
                if k.startswith("smsp__pcsamp_warps_issue_stalled_") and not k.endswith("_not_issued"):
                    v = num(r[i])
                    if v is not None:
                        stalls.append((v, k.replace("smsp__pcsamp_warps_issue_stalled_", "")))
            tot = sum(v for v, _ in stalls) or 1.0
            md += ["", "Warp-state samples (top 8, % of samples): " +
                   ", ".join(f"{k} {100 * v / tot:.1f}%" for v, k in sorted(stalls, reverse=True)[:8]), ""]
            if traffic_out and km and wkey:
                rd = to_bytes(r[h.index("dram__bytes_read.sum")], u[h.index("dram__bytes_read.sum")])
                wr = to_bytes(r[h.index("dram__bytes_write.sum")], u[h.index("dram__bytes_write.sum")])
                dur = num(r[h.index("gpu__time_duration.sum")])
                traffic.setdefault(km, {})[wkey] = {
                    "kernel": kn, "dram_bytes_per_launch": rd + wr, "dram_read": rd, "dram_write": wr,
                    "duration": dur, "duration_unit": u[h.index("gpu__time_duration.sum")],
                    "source": f"ncu --set full --clock-control none ({name}, launch {j}); "
                              f"summary in profiles/"}
    text = "\n".join(md)
    if md_out:
        with open(md_out, "a") as f:
            f.write(text + "\n")
    else:
        print(text)
    if traffic_out:
        with open(traffic_out, "w") as f:
            json.dump(traffic, f, indent=1, sort_keys=True)


if __name__ == "__main__":
    main()
