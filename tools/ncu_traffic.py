"""Per-launch DRAM traffic and pipe counters of every bench config's headline
kernel (and its exact kernel), in the exact launch configuration bench.py
times, from ncu -> profiles/ncu_traffic.json (keyed "<config>/<kernel key>").

  python tools/ncu_traffic.py                # orchestrate (on a GPU box): runs ncu per config
  python tools/ncu_traffic.py --drive C2     # (internal) the launches ncu profiles

bench.py reads the file for roofline.traffic (dram__bytes_read.sum +
dram__bytes_write.sum of one launch) and, for the ALU-bound median (C3), the
ALU-pipe instruction count behind its pipe-resolved roofline.  Each plan
launches twice (a warm-up, then the measured launch): ncu -k regex:perf_kernel
--launch-skip 1 --launch-count 1 per variant is emulated by recording every
launch and keeping the odd ones.  C4: one per-step launch of the 16384^2 grid
(bench's loop runs 200 of them).
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

METRICS = ["dram__bytes_read.sum", "dram__bytes_write.sum", "gpu__time_duration.sum", "smsp__inst_executed.sum",
           "smsp__inst_executed_pipe_alu.sum", "smsp__inst_executed_pipe_fma.sum",
           "sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active",
           "sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active", "sm__cycles_elapsed.avg.per_second",
           "lts__t_sector_hit_rate.pct"]


def key_of(app, r, scheme, rate, recon):
    return f"{app}{r}_{scheme}_{rate[0]}-{rate[1]}_{recon}"


def drive(cfg_name):
    import torch

    import paper_conf_cgo_maiercj18_b200 as kp
    import synth
    from bench import CONFIGS
    cfg = CONFIGS[cfg_name]
    app, W, H = cfg["app"], cfg["W"], cfg["H"]
    variants = [(cfg["scheme"], cfg["rate"], cfg["recon"]), ("none", (0, 1), "nn")]
    if app == "hotspot":
        T = torch.empty((H, W), device="cuda")
        P = torch.empty_like(T)
        synth.hotspot_band_device(cfg["seed"], W, H, 0, H, T.data_ptr(), P.data_ptr())
        o = torch.empty_like(T)
        for s, rt, rc in variants:
            with kp.Plan("hotspot", W, H, 1, s, rt, rc, iters=1, graph=0) as p:
                p.hotspot(T, P, o)
                p.hotspot(T, P, o)
                torch.cuda.synchronize()
            print(key_of(app, 1, s, rt, rc), flush=True)
        return
    u8 = app == "median"
    B = cfg["batch"]
    x = torch.empty((B, H, W), device="cuda", dtype=torch.uint8 if u8 else torch.float32)
    synth.image_device(cfg["cls"], cfg["seed"], W, H, B, x.data_ptr(), u8)
    y = torch.empty_like(x)
    for s, rt, rc in variants:
        with kp.Plan(app, W, H, cfg["r"], s, rt, rc, batch=B, granule_bytes=128) as p:
            p.run(x, y)
            p.run(x, y)
            torch.cuda.synchronize()
        print(key_of(app, cfg["r"], s, rt, rc), flush=True)


def main():
    if len(sys.argv) > 2 and sys.argv[1] == "--drive":
        drive(sys.argv[2])
        return
    from bench import CONFIGS
    out_path = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    res = {}
    for name in ("C1", "C2", "C3", "C4", "C5"):
        cmd = ["ncu", "--metrics", ",".join(METRICS), "--clock-control", "none", "--cache-control", "all",
               "-k", "regex:perf_kernel", "--csv", sys.executable, __file__, "--drive", name]
        p = subprocess.run(cmd, capture_output=True, text=True, cwd=ROOT)
        names = [ln.strip() for ln in p.stdout.splitlines() if ln.strip() and not ln.startswith(("==", '"'))]
        rows = list(csv.reader(io.StringIO("\n".join(ln for ln in p.stdout.splitlines() if ln.startswith('"')))))
        if not rows:
            print(name, "no ncu output:", p.stderr[-800:])
            continue
        hdr = rows[0]
        c = {h: i for i, h in enumerate(hdr)}
        per = {}
        for r in rows[1:]:
            per.setdefault(int(r[c["ID"]]), {})[r[c["Metric Name"]]] = float(r[c["Metric Value"]].replace(",", ""))
        ids = sorted(per)
        for k, nm in enumerate(names):
            m = per.get(ids[2 * k + 1]) if 2 * k + 1 < len(ids) else None
            if not m:
                continue
            res[f"{name}/{nm}"] = {
                "dram_read_bytes": m["dram__bytes_read.sum"], "dram_write_bytes": m["dram__bytes_write.sum"],
                "traffic": m["dram__bytes_read.sum"] + m["dram__bytes_write.sum"],
                "time_us_ncu": m["gpu__time_duration.sum"] / 1e3, "warp_inst": m["smsp__inst_executed.sum"],
                "warp_inst_pipe_alu": m["smsp__inst_executed_pipe_alu.sum"],
                "warp_inst_pipe_fma": m["smsp__inst_executed_pipe_fma.sum"],
                "pipe_alu_pct_of_peak": m["sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active"],
                "pipe_fma_pct_of_peak": m["sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active"],
                "sm_hz": m["sm__cycles_elapsed.avg.per_second"], "l2_hit_pct": m["lts__t_sector_hit_rate.pct"],
                "launch": f"bench.py {name} launch configuration, 2nd of 2 launches, ncu --cache-control all"}
            print(name, nm, res[f"{name}/{nm}"]["traffic"] / 1e6, "MB")
    res["_how"] = ("tools/ncu_traffic.py: ncu --metrics (dram bytes, time, pipe instruction counts) "
                   "--clock-control none --cache-control all, one measured launch per kernel")
    json.dump(res, open(out_path, "w"), indent=1, sort_keys=True)
    print("wrote", out_path)


if __name__ == "__main__":
    main()
