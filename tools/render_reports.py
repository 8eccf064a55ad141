"""Render the phase-profile and accuracy JSON lines (tools/phase_profile.py,
tools/accuracy_report.py) into the markdown summaries under profiles/.

  python tools/render_reports.py profiles/r02_phase_profile.jsonl profiles/r02_accuracy_fig18.jsonl
"""
import json
import sys


def phases_md(path):
    out = ["# Phase profile (B200 analogue of Figs 8/11/13/15/16; NEXT f4)", "",
           f"Source: `{path}` (tools/phase_profile.py, TRIDIAG_PHASE_STAMPS=1; clock64() on lane 0 of "
           "warp 0 of every CTA, first 4 units; cycles at ~1.9 GHz).  The stamps are one warp's "
           "latencies: phases of different warps / CTAs overlap, so they explain where a unit's time "
           "goes, not the kernel's throughput.", ""]
    rows = [json.loads(l) for l in open(path)]
    out += ["## Warp kernels (n <= 32 R): cycles per system group", "",
            "| dtype | n | algo | m | total | loads + in-lane fwd | tail chain | lane-level CR + inner | in-lane bwd | store |",
            "|---|---|---|---|---|---|---|---|---|---|"]
    for r in rows:
        if "phases" in r and "kernel" not in r:
            v = [round(p["cycles"]) for p in r["phases"].values()]
            out.append(f"| {r['dtype']} | {r['n']} | {r['algo']} | {r['m']} | {round(r['cycles_per_group'])} | "
                       + " | ".join(str(x) for x in v) + " |")
    out += ["", "## TMA CTA kernel (n > 32 R): cycles per system, steady state (systems 2-4 of each CTA)", ""]
    for r in rows:
        if r.get("kernel") == "tdg_cta_tma_kernel":
            st = r["steady"]
            out.append(f"- {r['dtype']} n={r['n']} S={r['S']} {r['algo']}: {round(st['cycles_per_system'])} cycles "
                       f"(first system {round(r['first_system']['cycles_per_system'])}): "
                       + ", ".join(f"{k} {round(v['cycles'])} ({100 * v['share']:.0f}%)" for k, v in st["phases"].items()))
    out += ["", "## Multi-launch paths: cycles per unit per pass", ""]
    for r in rows:
        if "launches" in r:
            out.append(f"- {r['dtype']} n={r['n']} S={r['S']} ({r['layout']}):")
            for L in r["launches"]:
                if "phases" in L:
                    out.append(f"  - launch {L['launch']} {L['pass']}: {round(L['cycles_per_unit'])} cycles/unit: "
                               + ", ".join(f"{k} {round(v['cycles'])}" for k, v in L["phases"].items()))
                else:
                    out.append(f"  - launch {L['launch']} `{L['kernel'][:48]}` ({L['units']} stamped units)")
    return "\n".join(out) + "\n"


def acc_md(path):
    rows = [json.loads(l) for l in open(path)]
    cols = ["cr", "pcr", "rd", "cr_pcr", "cr_rd", "cpu_ge_fp32", "cpu_gep_sgtsv"]

    def cell(v):
        if v["residual_max"] is None:
            return f"overflow ({v['nonfinite']}/512 non-finite)"
        s = f"{v['residual_max']:.1e} / {v['error_max']:.1e}"
        return s + (f" ({v['nonfinite']} nf)" if v["nonfinite"] else "")
    out = ["# Accuracy, fp32 (Fig 18, P:L1225-1240; SURVEY.md 8(c) R1/R2)", "",
           f"Source: `{path}` (tools/accuracy_report.py).  S = 512 systems per point.  Each cell: max "
           "residual ||Ax - d||_inf / max normwise error vs fp64 Thomas (finite systems), and the count "
           "of systems with a non-finite x.  KM(E) and DD stand in for the paper's fluid-simulation "
           "matrices (R19), CV is 'close values in all rows'.  CPU: the oracle's Thomas in fp32 (the "
           "paper's GE / MT) and LAPACK sgtsv (partial pivoting, the paper's GEP).", "",
           "| family | n | " + " | ".join(cols) + " |", "|---|---|" + "---|" * len(cols)]
    for r in rows:
        out.append(f"| {r['family']} | {r['n']} | " + " | ".join(cell(r[c]) for c in cols) + " |")
    out += ["", "As in the paper: on the dominant sets CR, PCR and CR+PCR are as accurate as GE, while RD "
            "and CR+RD overflow (fp32, n >= 64-128) or, on the weakly dominant KM(100), lose all accuracy; on "
            "close-value rows CR, PCR and CR+PCR lose accuracy (residuals up to 1e1 at n = 512), RD and "
            "CR+RD survive with residuals ~1e-3, and pivoting (sgtsv) is best."]
    return "\n".join(out) + "\n"


if __name__ == "__main__":
    ph, acc = sys.argv[1], sys.argv[2]
    open(ph.replace(".jsonl", ".md"), "w").write(phases_md(ph))
    open(acc.replace(".jsonl", ".md"), "w").write(acc_md(acc))
