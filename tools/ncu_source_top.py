"""Top stall-sampled SASS lines / CUDA source lines of one kernel in an .ncu-rep.
usage: ncu_source_top.py rep.ncu-rep [kernel-index] [n]"""
import csv
import io
import subprocess
import sys

rep = sys.argv[1]
idx = int(sys.argv[2]) if len(sys.argv) > 2 else 0
n = int(sys.argv[3]) if len(sys.argv) > 3 else 25


def f(x):
    try:
        return float(x)
    except ValueError:
        return 0.0


for view in ("sass", "cuda"):
    out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", view,
                          "--launch-skip", str(idx), "--launch-count", "1"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr_i = next(i for i, r in enumerate(rows) if r and r[0] in ("Address", "Line", "#"))
    hdr = rows[hdr_i]
    col = {h: i for i, h in enumerate(hdr)}
    data = [r for r in rows[hdr_i + 1:] if len(r) == len(hdr)]
    key = "Warp Stall Sampling (All Samples)"
    tot = sum(f(r[col[key]]) for r in data)
    print(f"== {view}: {tot:.0f} samples")
    for r in sorted(data, key=lambda r: -f(r[col[key]]))[:n]:
        src = r[col["Source"]].strip()[:110]
        print(f"{f(r[col[key]]) / max(tot, 1) * 100:5.1f}%  {r[0]:>8}  {src}")
