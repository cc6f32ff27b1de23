"""Turn one tools/profile_round.sh output directory into the committed text
evidence under profiles/<tag>/ (bench lines, launch list, ncu summaries,
per-variant DRAM bytes).  usage: collect_profiles.py gpurun_out/prof profiles/r01"""
import collections
import csv
import io
import json
import os
import shutil
import subprocess
import sys

src, dst = sys.argv[1], sys.argv[2]
os.makedirs(dst, exist_ok=True)

for f in sorted(os.listdir(src)):
    if f.startswith("bench_") and f.endswith(".json"):
        shutil.copy(os.path.join(src, f), os.path.join(dst, f))

# launch list (shares of the bench step)
lc = os.path.join(src, "launches_bench_c2.csv")
if os.path.exists(lc):
    rows = [r for r in csv.reader(open(lc)) if r]
    hdr = next(r for r in rows if r[0] == "ID")
    ki, mi, vi = hdr.index("Kernel Name"), hdr.index("Metric Name"), hdr.index("Metric Value")
    t = collections.OrderedDict()
    for r in rows[rows.index(hdr) + 1:]:
        if len(r) == len(hdr) and r[mi] == "gpu__time_duration.sum":
            n, s = t.get(r[ki], (0, 0.0))
            t[r[ki]] = (n + 1, s + float(r[vi].replace(",", "")))
    tot = sum(s for _, s in t.values())
    with open(os.path.join(dst, "launch_list_bench_c2.txt"), "w") as fo:
        fo.write("ncu --metrics gpu__time_duration.sum --clock-control none: "
                 "python bench.py --steps 2 --warmup 3 --no-variants --no-cpu\n"
                 "(cold-cache, serialised launches: compare shares, not absolute times; "
                 "times in ns)\n")
        for k, (n, s) in sorted(t.items(), key=lambda kv: -kv[1][1]):
            fo.write(f"{n:3d} launches {s:12.1f}   {100 * s / tot:5.1f}%  {k[:100]}\n")
    shutil.copy(lc, os.path.join(dst, "launches_bench_c2.csv"))

# --set full summaries
here = os.path.dirname(os.path.abspath(__file__))
for rep, name in [("ncu_full_headline", "ncu_full_headline_gaussian5_row12_li.txt"),
                  ("ncu_full_exact", "ncu_full_exact_gaussian5.txt"),
                  ("ncu_full_tb8_row", "ncu_full_hotspot_tb8_row12.txt"),
                  ("ncu_full_tb8_exact", "ncu_full_hotspot_tb8_exact.txt")]:
    p = os.path.join(src, rep + ".ncu-rep")
    if os.path.exists(p):
        out = subprocess.run([sys.executable, os.path.join(here, "ncu_summary.py"), p],
                             capture_output=True, text=True).stdout
        details = subprocess.run(["ncu", "-i", p, "--page", "details"], capture_output=True, text=True).stdout
        with open(os.path.join(dst, name), "w") as fo:
            fo.write(f"ncu --set full --import-source on --clock-control none ({rep}.ncu-rep)\n")
            fo.write(out + "\n---- details page ----\n" + details)

# per-variant DRAM bytes
for v in ["all", "c1", "c3", "c5"]:
    p, lg = os.path.join(src, f"ncu_variants_{v}.csv"), os.path.join(src, f"ncu_variants_{v}.log")
    if os.path.exists(p):
        shutil.copy(p, os.path.join(dst, f"ncu_variants_{v}.csv"))
        if os.path.exists(lg):
            shutil.copy(lg, os.path.join(dst, f"ncu_variants_{v}.log"))
print("wrote", sorted(os.listdir(dst)))
