"""NEXT-2: the paper's sensitivity and parameter studies on synthetic stand-ins,
through the GPU path (libkperf) -- Fig. 6/7/8 (error per image class and per
scheme) and Fig. 9 (tile shape vs runtime).

  python tools/study.py [--out gpurun_out/study.json] [--images 8]   (r01 results: profiles/r01/study.txt)

Images: 1024 x 1024 (the paper's size), classes flat /
natural / pattern (Fig. 7's flat / photo / pattern), seeds
0x5EED3000 + class*100 + i.  Error = MRE of the perforated output against the
exact kernel's.  Times: CUDA events, batch of all images.
"""
import argparse
import json
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
import synth  # noqa: E402

VARIANTS = [("Rows1:NN", "row", (1, 2), "nn", {}), ("Rows2:NN", "row", (3, 4), "nn", {}),
            ("Rows1:LI", "row", (1, 2), "li", {}), ("Stencil1:NN", "stencil1", (0, 1), "nn", {})]
APPS = [("gaussian", 1), ("inversion", 0), ("median", 1)]


def time_ms(fn, reps=20):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps):
        fn()
    b.record()
    b.synchronize()
    return a.elapsed_time(b) / reps


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=os.path.join(ROOT, "gpurun_out", "study.json"))
    ap.add_argument("--images", type=int, default=8)
    a = ap.parse_args()
    W = H = 1024
    n = a.images
    res = {"images_per_class": n, "size": [W, H], "errors": {}, "times_ms": {}, "tile_sweep": {}}
    for app, r in APPS:
        u8 = app == "median"
        dt = torch.uint8 if u8 else torch.float32
        for ci, cls in enumerate(("flat", "natural", "pattern")):
            x = torch.empty((n, H, W), dtype=dt, device="cuda")
            synth.image_device(cls, 0x5EED3000 + 100 * ci, W, H, n, x.data_ptr(), u8)
            ex = torch.empty_like(x)
            with kp.Plan(app, W, H, r, batch=n) as pe:
                pe.run(x, ex)
                if ci == 1:
                    res["times_ms"][f"{app}:exact"] = time_ms(lambda: pe.run(x, ex))
            for name, scheme, rate, recon, keys in VARIANTS:
                y = torch.empty_like(x)
                with kp.Plan(app, W, H, r, scheme, rate, recon, batch=1, **keys) as p:
                    errs = []
                    for i in range(n):
                        p.run(x[i], y[i])
                        errs.append(p.error(ex[i], y[i])[0])
                res["errors"][f"{app}:{cls}:{name}"] = errs
                if ci == 1:
                    with kp.Plan(app, W, H, r, scheme, rate, recon, batch=n, **keys) as pb:
                        res["times_ms"][f"{app}:{name}"] = time_ms(lambda: pb.run(x, y))
            if ci == 1:  # Fig. 9: tile shape (work-group size) vs runtime, exact and perforated
                for tw, th in ((16, 16), (32, 8), (64, 4), (128, 2), (256, 1), (16, 32), (16, 64)):
                    with kp.Plan(app, W, H, r, "stencil1", (0, 1), "nn", batch=n, tile1_w=tw, tile1_h=th) as ps:
                        res["tile_sweep"][f"{app}:Stencil1:{tw}x{th}"] = time_ms(lambda: ps.run(x, y))
                for seg in (8, 32, 128, 512):
                    with kp.Plan(app, W, H, r, batch=n, tile_h=seg) as pe2, \
                            kp.Plan(app, W, H, r, "row", (1, 2), "nn", batch=n, tile_h=seg) as pr:
                        res["tile_sweep"][f"{app}:exact:seg{seg}"] = time_ms(lambda: pe2.run(x, ex))
                        res["tile_sweep"][f"{app}:Rows1:seg{seg}"] = time_ms(lambda: pr.run(x, y))
    os.makedirs(os.path.dirname(a.out), exist_ok=True)
    json.dump(res, open(a.out, "w"), indent=1)
    lines = [f"{'app:class:variant':36s} {'median MRE':>10s} {'q1':>8s} {'q3':>8s} {'max':>8s}"]
    for k, v in res["errors"].items():
        q = np.percentile(v, [25, 50, 75, 100])
        lines.append(f"{k:36s} {q[1]:10.5f} {q[0]:8.5f} {q[2]:8.5f} {q[3]:8.5f}")
    lines.append("")
    for k, v in res["times_ms"].items():
        lines.append(f"time {k:30s} {v * 1e3:9.1f} us ({n} x 1024^2)")
    for k, v in res["tile_sweep"].items():
        lines.append(f"tile {k:30s} {v * 1e3:9.1f} us")
    open(a.out.replace(".json", ".txt"), "w").write("\n".join(lines) + "\n")
    print("\n".join(lines))


if __name__ == "__main__":
    main()
