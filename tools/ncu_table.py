"""Print per-variant ncu metrics from a --csv log written over tools/ncu_driver.py
(measured launches = odd IDs).  usage: ncu_table.py metrics.csv driver.log px_per_launch"""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
names = [l.strip() for l in open(sys.argv[2]) if l.strip() and not l.startswith("==")]
px = float(sys.argv[3])
hdr, recs = None, {}
for r in rows:
    if r and r[0] == "ID":
        hdr = r
        continue
    if hdr and len(r) == len(hdr):
        d = dict(zip(hdr, r))
        recs.setdefault(int(d["ID"]), {})[d["Metric Name"]] = float(d["Metric Value"].replace(",", ""))
for i, n in enumerate(names):
    m = recs.get(2 * i + 1, {})
    print(f"{n:28s} rd {m.get('dram__bytes_read.sum', 0) / 1e6:8.1f}MB wr {m.get('dram__bytes_write.sum', 0) / 1e6:8.1f}MB "
          f"t {m.get('gpu__time_duration.sum', 0) / 1e3:7.1f}us inst/128px {m.get('smsp__inst_executed.sum', 0) / (px / 128):6.1f} "
          f"warps% {m.get('sm__warps_active.avg.pct_of_peak_sustained_active', 0):5.1f}")
