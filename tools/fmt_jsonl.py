"""Condense JSON-lines sweep output (tools/tune.py, tools/sweep.py) into one
short text line per point; non-JSON lines pass through."""
import json
import sys

for line in sys.stdin:
    try:
        r = json.loads(line)
    except Exception:
        print(line.rstrip())
        continue
    if "frac" in r and "us" in r:
        print(r.get("dtype"), r.get("n"), r.get("algo"), r.get("m"), round(r["us"], 1), round(r["frac"], 3))
    elif "frac_of_peak" in r:
        mf = r.get("model_frac")
        acc = (r.get("acc") or {}).get("max_err")
        print(r.get("config"), r.get("dtype"), r.get("grid") or r.get("n"), r.get("S"), r.get("algo"),
              r.get("m"), round(r["frac_of_peak"], 3), mf and round(mf, 3), acc)
    else:
        print(line.rstrip()[:300])
