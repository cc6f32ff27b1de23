"""TILE_H (segment height) sweep over the BASELINE workloads: ms per launch
for auto (0) and fixed segment heights.  usage: sweep_tile_h.py"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
import synth  # noqa: E402

HS = (0, 24, 32, 48, 64, 96, 128)


def t(fn, reps=20):
    for _ in range(3):
        fn()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    e1.synchronize()
    return e0.elapsed_time(e1) / reps


def sweep(name, W, H, B, u8, variants):
    x = torch.empty((B, H, W), device="cuda", dtype=torch.uint8 if u8 else torch.float32)
    synth.image_device("natural", 0x5EED0011, W, H, B, x.data_ptr(), u8)
    y = torch.empty_like(x)
    for app, r, s, rate, rc in variants:
        row = []
        for th in HS:
            keys = dict(batch=B)
            if th:
                keys["tile_h"] = th
            with kp.Plan(app, W, H, r, s, rate, rc, **keys) as p:
                row.append(t(lambda: p.run(x, y)))
        print(f"{name} {app}{r} {s} {rate} {rc}: " + "  ".join(f"{h or 'auto'}:{m:.4f}" for h, m in zip(HS, row)),
              flush=True)
    del x, y


sweep("C2", 4096, 4096, 8, False, [("gaussian", 2, "none", (0, 1), "nn"), ("gaussian", 2, "row", (1, 2), "li"),
                                   ("gaussian", 2, "row", (1, 4), "nn"), ("gaussian", 2, "row", (3, 4), "li"),
                                   ("sobel", 1, "none", (0, 1), "nn"), ("sobel", 1, "row", (1, 2), "nn"),
                                   ("gaussian", 2, "col", (1, 2), "nn"), ("gaussian", 2, "checker", (1, 2), "nn"),
                                   ("gaussian", 2, "checker", (1, 4), "li"), ("gaussian", 2, "checker", (3, 4), "li")])
sweep("C3", 8192, 8192, 4, True, [("median", 1, "none", (0, 1), "nn"), ("median", 1, "col", (1, 2), "nn")])
sweep("C5", 3840, 2160, 16, False, [("gauss_sobel", 2, "none", (0, 1), "nn"), ("gauss_sobel", 2, "row", (1, 2), "li")])
sweep("C1", 512, 512, 512, False, [("gaussian", 2, "none", (0, 1), "nn"), ("gaussian", 2, "row", (1, 2), "li")])
