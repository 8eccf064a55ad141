"""Summarise `nvcc -Xptxas -v` output: kernel, registers, spills, stack."""
import re
import subprocess
import sys

txt = sys.stdin.read()
rows = []
cur = None
for line in txt.splitlines():
    m = re.search(r"Function properties for (\S+)", line)
    if m:
        cur = {"name": m.group(1)}
        continue
    if cur is None:
        continue
    m = re.search(r"(\d+) bytes stack frame, (\d+) bytes spill stores, (\d+) bytes spill loads", line)
    if m:
        cur["stack"], cur["sst"], cur["sld"] = map(int, m.groups())
        continue
    m = re.search(r"Used (\d+) registers", line)
    if m:
        cur["regs"] = int(m.group(1))
        if "ilog2c" not in cur["name"]:
            rows.append(cur)
        cur = None
for r in rows:
    try:
        dem = subprocess.run(["c++filt", r["name"]], capture_output=True, text=True).stdout.strip()
    except Exception:
        dem = r["name"]
    dem = re.sub(r"\(.*", "", dem).replace("void tdg::", "")
    print(f"{r['regs']:4d} regs  spill {r.get('sst',0):4d}/{r.get('sld',0):4d}  stack {r.get('stack',0):4d}  {dem}")
