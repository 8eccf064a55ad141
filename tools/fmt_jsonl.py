import sys,json
for l in sys.stdin:
  try: r=json.loads(l)
  except Exception: print(l.strip()); continue
  if "frac" in r: print(r.get("dtype"),r["n"],r["algo"],r["m"],round(r["us"],1),round(r["frac"],3))
  elif "frac_of_peak" in r: print(r["config"],r["dtype"],r["n"],r["S"],r["algo"],r.get("m"),round(r["frac_of_peak"],3), r.get("model_frac") and round(r["model_frac"],3), r.get("acc",{}).get("max_err"))
  else: print(l.strip()[:300])
