"""Markdown summary of tools/tune.py output (plan R x prefetch x m sweep)."""
import collections
import json
import sys

rows = [json.loads(l) for l in open(sys.argv[1]) if l.strip()]
tab = collections.defaultdict(dict)
for r in rows:
    if "error" in r:
        continue
    n = r["n"]
    R = r.get("TRIDIAG_WARP_R")
    R = int(R) if R is not None else None
    if R is not None and not (R <= n and n // R <= 32):
        R = None
    key = (r["dtype"], n, r["S"], r["algo"], r["m"])
    tab[key][(R or "default", r.get("TRIDIAG_PREFETCH"))] = r["frac"]
print("| dtype | n | S | algo | m | best (R, prefetch) | best % of measured peak | all (R/prefetch: %) |")
print("|---|---|---|---|---|---|---|---|")
for key in sorted(tab, key=lambda k: (k[0], k[1], k[2], k[3], k[4])):
    d = tab[key]
    best = max(d.items(), key=lambda kv: kv[1])
    allv = " ".join(f"{k[0]}/{k[1]}:{v*100:.0f}" for k, v in sorted(d.items(), key=lambda kv: str(kv[0])))
    print(f"| {key[0]} | {key[1]} | {key[2]} | {key[3]} | {key[4]} | {best[0]} | {best[1]*100:.1f} | {allv} |")
