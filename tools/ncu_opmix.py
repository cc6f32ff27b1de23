"""Executed-instruction mix (warp-level) of one kernel in an .ncu-rep, by opcode.
usage: ncu_opmix.py rep.ncu-rep [top]"""
import collections
import csv
import io
import subprocess
import sys

out = subprocess.run(["ncu", "-i", sys.argv[1], "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
hi = next(i for i, r in enumerate(rows) if r and r[0] == "Address")
hdr = rows[hi]
col = {h: i for i, h in enumerate(hdr)}
c = collections.Counter()
tot = 0.0
for r in rows[hi + 1:]:
    if len(r) != len(hdr):
        continue
    t = r[col["Source"]].strip()
    if not t:
        continue
    if t.startswith("@"):
        t = t.split(None, 1)[1]
    n = float(r[col["Instructions Executed"]] or 0)
    c[t.split()[0].split(".")[0]] += n
    tot += n
print(f"total warp instructions: {tot:.0f}")
for op, n in c.most_common(int(sys.argv[2]) if len(sys.argv) > 2 else 30):
    print(f"  {op:12s} {n:12.0f} {n / tot * 100:5.1f}%")
