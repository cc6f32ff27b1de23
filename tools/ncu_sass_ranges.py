"""Stall samples of an ncu --page source (sass) CSV, grouped into contiguous
address ranges with the dominant stall reasons -- locates which loop of a
kernel (producer / consumer waits / compute) the samples fall in.
usage: ncu_sass_ranges.py rep.ncu-rep [range-size]"""
import csv
import io
import subprocess
import sys

rep = sys.argv[1]
step = int(sys.argv[2]) if len(sys.argv) > 2 else 100
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
hi = next(i for i, r in enumerate(rows) if r and r[0] == "Address")
hdr = rows[hi]
data = [r for r in rows[hi + 1:] if len(r) == len(hdr)]
st = [j for j, h in enumerate(hdr) if h.startswith("stall_")]


def f(x):
    try:
        return float(x)
    except ValueError:
        return 0.0


tot = sum(f(r[2]) for r in data) or 1
for a in range(0, len(data), step):
    blk = data[a:a + step]
    s = sum(f(r[2]) for r in blk)
    if s / tot < 0.01:
        continue
    reasons = sorted(((sum(f(r[j]) for r in blk), hdr[j][6:]) for j in st), reverse=True)[:4]
    ops = {}
    for r in blk:
        op = r[1].split()[1 if r[1].lstrip().startswith("@") else 0].split(".")[0] if r[1].strip() else ""
        ops[op] = ops.get(op, 0) + f(r[2])
    top_ops = sorted(ops.items(), key=lambda t: -t[1])[:4]
    print(f"[{a:5d}-{a + len(blk) - 1:5d}] {s / tot * 100:5.1f}%  stalls " +
          ", ".join(f"{n}:{v / tot * 100:.1f}" for v, n in reasons) + "  ops " +
          ", ".join(f"{o}:{v / tot * 100:.1f}" for o, v in top_ops))
