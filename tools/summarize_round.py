"""Summarise a measurement pass (tools/profile_round2.sh output directory) into
a markdown file next to it: bench lines per config, the C2 variant table, the
3-class / 1-px sweep, per-launch ncu DRAM bytes of every variant vs the exact
kernel, and the roofline numbers recomputed from the files themselves.

  python tools/summarize_round.py profiles/r02 > profiles/r02/SUMMARY.md
"""
import csv
import json
import os
import sys


def load(d, name):
    p = os.path.join(d, name)
    if not os.path.exists(p):
        return None
    txt = open(p).read().strip().splitlines()
    for line in reversed(txt):
        if line.startswith("{"):
            return json.loads(line)
    return None


def ncu_rows(path):
    """(variant name in launch order, metrics of the measured (2nd) launch)"""
    if not os.path.exists(path):
        return []
    lines = open(path).read().splitlines()
    rows = list(csv.reader([ln for ln in lines if ln.startswith('"')]))
    if not rows:
        return []
    hdr = rows[0]
    c = {h: i for i, h in enumerate(hdr)}
    per = {}
    for r in rows[1:]:
        per.setdefault(int(r[c["ID"]]), {})[r[c["Metric Name"]]] = float(r[c["Metric Value"]].replace(",", ""))
    logp = path.replace(".csv", ".log")
    names = [ln.strip() for ln in open(logp).read().splitlines() if ln.strip() and not ln.startswith("==")] \
        if os.path.exists(logp) else []
    ids = sorted(per)
    out = []
    for k, nm in enumerate(names):
        if 2 * k + 1 < len(ids):
            out.append((nm, per[ids[2 * k + 1]]))
    return out


def main():
    d = sys.argv[1]
    print(f"# Measurement summary: `{d}`\n")
    print("Bench lines (`python bench.py --config C`; driver contract, CUDA events, inputs > L2):\n")
    print("| config | workload | ms/step | value | x exact | error | roofline (bound, achieved/peak = frac) | "
          "ncu traffic/launch | CPU oracle 1 core / all cores | e2e |")
    print("|---|---|---|---|---|---|---|---|---|---|")
    for c in ("C1", "C2", "C3", "C4", "C5"):
        b = load(d, f"bench_{c}.json")
        if not b:
            continue
        rf = b["roofline"]
        cb = b.get("cpu_baseline", {})
        allc = cb.get("all_cores", {})
        e2e = b.get("e2e", {}).get("value") if isinstance(b.get("e2e"), dict) else None
        tr = rf.get("traffic")
        print(f"| {c} | {b['config']['workload']} | {b['ms_per_step']:.4f} | {b['value']:.4g} {b['unit']} | "
              f"{b.get('speedup_vs_exact', 0):.3f} | {b.get('error', {}).get('metric')} {b.get('error', {}).get('value', 0):.4g} | "
              f"{rf['bound']} {rf['achieved']:.4g}/{rf['peak']:.4g} {rf['unit']} = {rf['frac']:.3f} | "
              f"{(tr / 1e6):.1f} MB |" if tr else "n/a |", end="")
        print(f" {cb.get('value', 0):.3g} / {allc.get('value', 0):.3g} ({allc.get('cores')} cores) | "
              f"{e2e:.4g} |" if e2e else f" {cb.get('value', 0):.3g} / {allc.get('value', 0):.3g} | n/a |")
    b = load(d, "bench_C2.json")
    if b and b.get("variants"):
        print("\nC2 variants (8 x 4096² fp32, 128-B cells, natural class; ms per launch):\n")
        print("| app | scheme | rate | recon | µs | x exact | error | HBM frac |")
        print("|---|---|---|---|---|---|---|---|")
        for v in b["variants"]:
            print(f"| {v['app']}{v['r']} | {v['scheme']}{' ' + str(v.get('tile')) if v.get('tile') else ''} | "
                  f"{v['rate'][0]}/{v['rate'][1]} | {v['recon']} | {v['ms'] * 1e3:.1f} | {v['speedup']:.3f} | "
                  f"{v['error']:.4g} | {v['frac']:.3f} |")
    sw = load(d, "sweep_c2.json")
    if sw:
        print("\nC2 sweep: input class x cell width (`bench.py --sweep`; G = 4 B is the pixel-granular cell):\n")
        print("| class | app | scheme | G bytes | rate | recon | µs | x exact | error |")
        print("|---|---|---|---|---|---|---|---|---|")
        for v in sw["sweep"]:
            print(f"| {v['class']} | {v['app']}{v['r']} | {v['scheme']} | {v['granule_bytes'] or '-'} | "
                  f"{v['rate'][0]}/{v['rate'][1]} | {v['recon']} | {v['ms'] * 1e3:.1f} | {v['speedup']:.3f} | "
                  f"{v['error']:.4g} |")
    for tag, fname in (("128-B cells", "ncu_variants_all.csv"), ("1-px cells (G = 4 B)", "ncu_variants_all_g1px.csv"),
                       ("C3 median", "ncu_variants_c3all.csv"), ("C5 fused", "ncu_variants_c5.csv"),
                       ("C1", "ncu_variants_c1.csv")):
        rows = ncu_rows(os.path.join(d, fname))
        if not rows:
            continue
        ex = {}
        for nm, m in rows:
            if "_none_" in nm:
                ex[nm.split("_")[0]] = m["dram__bytes_read.sum"]
        print(f"\nncu DRAM reads per launch, {tag} (batch 2; `north_star` target: read / exact <= kept fraction):\n")
        print("| variant | DRAM read MB | write MB | read / exact | kept fraction | time µs (ncu) |")
        print("|---|---|---|---|---|---|")
        for nm, m in rows:
            app = nm.split("_")[0]
            rd = m["dram__bytes_read.sum"]
            parts = nm.split("_")
            kept = 1.0
            if len(parts) >= 3 and parts[1] != "none" and "-" in parts[2]:
                a, bb = parts[2].split("-")
                kept = 1 - int(a) / int(bb)
            ratio = rd / ex[app] if app in ex and ex[app] else float("nan")
            print(f"| {nm} | {rd / 1e6:.1f} | {m['dram__bytes_write.sum'] / 1e6:.1f} | {ratio:.3f} | {kept:.3f} | "
                  f"{m['gpu__time_duration.sum'] / 1e3:.1f} |")
    tj = os.path.join(d, "ncu_traffic.json")
    if os.path.exists(tj):
        t = json.load(open(tj))
        print("\nPer-launch ncu counters in each bench config's own launch configuration (`tools/ncu_traffic.py`):\n")
        print("| config/kernel | DRAM read MB | write MB | traffic MB | warp inst | ALU-pipe inst | ALU pipe % | L2 hit % |")
        print("|---|---|---|---|---|---|---|---|")
        for k, v in sorted(t.items()):
            if k.startswith("_"):
                continue
            print(f"| {k} | {v['dram_read_bytes'] / 1e6:.1f} | {v['dram_write_bytes'] / 1e6:.1f} | "
                  f"{v['traffic'] / 1e6:.1f} | {v['warp_inst']:.4g} | {v['warp_inst_pipe_alu']:.4g} | "
                  f"{v['pipe_alu_pct_of_peak']:.1f} | {v['l2_hit_pct']:.1f} |")
    for t in ("memcheck", "racecheck", "synccheck"):
        p = os.path.join(d, f"sanitizer_{t}.log")
        if os.path.exists(p):
            last = [ln for ln in open(p).read().splitlines() if "SUMMARY" in ln]
            print(f"\ncompute-sanitizer {t}: {last[-1].strip('= ') if last else 'see log'}")


if __name__ == "__main__":
    main()
