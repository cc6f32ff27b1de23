"""Print a bench.py JSON line (and its C2 variants) as a compact table.
usage: bench_table.py bench.json [bench2.json]  (two files: side by side ms)"""
import json
import sys


def load(f):
    return json.loads(open(f).read().strip().splitlines()[-1])


ds = [load(f) for f in sys.argv[1:]]
d = ds[0]
r = d.get("roofline", {})
print(d["config"].get("workload"), "| value", round(d["value"]), d["unit"], "| ms", round(d["ms_per_step"], 4),
      "| frac", round(r.get("frac", 0), 3), "| frac_mix", r.get("frac_mix"), "| speedup", d.get("speedup_vs_exact"))
vs = [x.get("variants", []) for x in ds]
for i, v in enumerate(vs[0]):
    cols = [f"{w[i]['ms']:.4f}" for w in vs if i < len(w)]
    print(f"  {v['app']:9s} {v['scheme']:8s} {str(v['rate']):7s} {v['recon']:3s} ms " + " -> ".join(cols) +
          f"  spd {vs[-1][i]['speedup']:.3f} fmix {vs[-1][i].get('frac_mix', 0):.3f}")
