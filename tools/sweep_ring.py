"""Ring depth x segment height sweep for the cell-loader (column / checkerboard)
C2 variants: ms per launch (CUDA events, 8 x 4096^2 fp32 frames, median of
ROUNDS interleaved rounds).  Used to pick the auto ring depth (kperf.cu).
usage: sweep_ring.py [col|checker|row] [ROUNDS]"""
import itertools
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
import synth  # noqa: E402

scheme = sys.argv[1] if len(sys.argv) > 1 else "col"
rounds = int(sys.argv[2]) if len(sys.argv) > 2 else 3
W = H = 4096
B = 8
x = torch.empty((B, H, W), device="cuda")
synth.image_device("natural", 0x5EED0011, W, H, B, x.data_ptr(), False)
y = torch.empty_like(x)


def t(p, reps=10):
    for _ in range(2):
        p.run(x, y)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        p.run(x, y)
    e1.record()
    e1.synchronize()
    return e0.elapsed_time(e1) / reps * 1000


variants = [(a, r, scheme, rate, rc) for a, r in (("gaussian", 2), ("sobel", 1))
            for rate in ((1, 2), (1, 4), (3, 4)) for rc in ("nn", "li")]
if scheme == "row":
    variants += [("gaussian", 2, "none", (0, 1), "nn"), ("sobel", 1, "none", (0, 1), "nn")]
rings = {"col": (0, 4, 8), "checker": (0, 8, 16), "row": (0, 16)}[scheme]
ths = (0, 32, 64) if scheme != "row" else (0, 16, 24, 32, 40, 48)
if len(sys.argv) > 3:  # explicit lists: sweep_ring.py SCHEME ROUNDS rings ths (comma separated)
    rings = tuple(int(v) for v in sys.argv[3].split(","))
    ths = tuple(int(v) for v in sys.argv[4].split(","))
res = {}
for _ in range(rounds):
    for v, ring, th in itertools.product(variants, rings, ths):
        keys = dict(batch=B)
        if ring:
            keys["ring"] = ring
        if th:
            keys["tile_h"] = th
        try:
            with kp.Plan(v[0], W, H, v[1], v[2], v[3], v[4], **keys) as p:
                res.setdefault((v, ring, th), []).append(t(p))
        except Exception as e:  # noqa: BLE001
            res.setdefault((v, ring, th), []).append(float("nan"))
            print(v, ring, th, e, file=sys.stderr)
hdr = "variant".ljust(28) + "".join(f"r{ring}/h{th}".rjust(10) for ring, th in itertools.product(rings, ths))
print(hdr)
for v in variants:
    row = f"{v[0]}{v[1]} {v[2]} {v[3][0]}/{v[3][1]} {v[4]}".ljust(28)
    for ring, th in itertools.product(rings, ths):
        xs = sorted(res[(v, ring, th)])
        row += f"{xs[len(xs) // 2]:10.1f}"
    print(row, flush=True)
