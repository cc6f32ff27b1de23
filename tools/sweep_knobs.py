"""Sweep performance-only plan keys (RING, TILE_H, PRODUCER, LOADER) for one
C2 variant; prints ms per launch (CUDA events, 8 x 4096^2 fp32 frames).
usage: sweep_knobs.py [app r scheme num den recon]"""
import itertools
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
import synth  # noqa: E402

a = sys.argv[1:] or ["gaussian", "2", "row", "1", "2", "li"]
app, r, scheme, num, den, recon = a[0], int(a[1]), a[2], int(a[3]), int(a[4]), a[5]
W = H = 4096
B = 8
x = torch.empty((B, H, W), device="cuda")
synth.image_device("natural", 0x5EED0011, W, H, B, x.data_ptr(), False)
y = torch.empty_like(x)


def t(p, reps=20):
    for _ in range(3):
        p.run(x, y)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        p.run(x, y)
    e1.record()
    e1.synchronize()
    return e0.elapsed_time(e1) / reps


for ring, th in itertools.product((0, 8, 16, 32), (0, 32, 64, 128, 256)):
    keys = dict(batch=B)
    if ring:
        keys["ring"] = ring
    if th:
        keys["tile_h"] = th
    try:
        with kp.Plan(app, W, H, r, scheme, (num, den), recon, **keys) as p:
            print(f"ring {ring:3d} tile_h {th:4d}: {t(p):.4f} ms", flush=True)
    except Exception as e:  # noqa: BLE001
        print(f"ring {ring:3d} tile_h {th:4d}: {e}")
