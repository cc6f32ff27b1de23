"""A/B timing of experiment builds of libkperf.so on C2-sized inputs.
usage: [AB_KEYS='{"producer": 2}'] ab.py [--set row|all|col|checker|median|c5] lib1.so [lib2.so[@{"ring": 8}] ...]
Each library runs in its own process (KPERF_LIB); the libraries alternate
over ROUNDS rounds and the per-variant median is printed (ms per launch,
8 x 4096^2 fp32 frames; median: 4 x 8192^2 u8; c5: 16 x 3840x2160)."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SETS = {
    "row": [("gaussian", 2, "none", 0, 1, "nn"), ("gaussian", 2, "row", 1, 2, "li"), ("gaussian", 2, "row", 1, 2, "nn"),
            ("gaussian", 2, "row", 3, 4, "li"), ("sobel", 1, "row", 1, 2, "li"), ("sobel", 1, "none", 0, 1, "nn")],
    "col": [("gaussian", 2, "col", 1, 2, "li"), ("gaussian", 2, "col", 1, 4, "nn"), ("sobel", 1, "col", 1, 2, "nn")],
    "checker": [("gaussian", 2, "checker", 1, 2, "li"), ("gaussian", 2, "checker", 1, 2, "nn"),
                ("gaussian", 2, "checker", 1, 4, "li"), ("gaussian", 2, "checker", 1, 4, "nn"),
                ("gaussian", 2, "checker", 3, 4, "li"), ("gaussian", 2, "checker", 3, 4, "nn"),
                ("sobel", 1, "checker", 1, 4, "nn"), ("sobel", 1, "checker", 1, 2, "li")],
    "median": [("median", 1, "none", 0, 1, "nn"), ("median", 1, "col", 1, 2, "nn"), ("median", 1, "col", 1, 4, "nn"),
               ("median", 1, "col", 3, 4, "nn"), ("median", 1, "row", 1, 2, "nn")],
    "c5": [("gauss_sobel", 2, "none", 0, 1, "nn"), ("gauss_sobel", 2, "row", 1, 2, "li")],
    "c1": [("gaussian", 2, "none", 0, 1, "nn", 512, 512, 512), ("gaussian", 2, "row", 1, 2, "li", 512, 512, 512),
           ("sobel", 1, "row", 1, 2, "nn", 512, 512, 512)],
}
SETS["row34"] = [("gaussian", 2, "row", 3, 4, "nn"), ("gaussian", 2, "row", 3, 4, "li"), ("sobel", 1, "row", 3, 4, "nn"),
                 ("sobel", 1, "row", 3, 4, "li"), ("gaussian", 2, "none", 0, 1, "nn"), ("sobel", 1, "none", 0, 1, "nn")]
SETS["hotspot"] = [("hotspot", 1, "none", 0, 1, "nn"), ("hotspot", 1, "row", 1, 2, "li"), ("hotspot", 1, "row", 1, 2, "nn")]
SETS["colchk"] = [("gaussian", 2, "col", 1, 2, "li"), ("gaussian", 2, "col", 1, 2, "nn"), ("gaussian", 2, "col", 1, 4, "li"),
                  ("gaussian", 2, "col", 1, 4, "nn"), ("gaussian", 2, "col", 3, 4, "li"), ("gaussian", 2, "col", 3, 4, "nn"),
                  ("gaussian", 2, "checker", 1, 2, "li"), ("gaussian", 2, "checker", 1, 2, "nn"),
                  ("gaussian", 2, "checker", 3, 4, "li"), ("gaussian", 2, "checker", 3, 4, "nn"),
                  ("sobel", 1, "col", 1, 2, "nn"), ("sobel", 1, "col", 1, 4, "li"), ("sobel", 1, "checker", 3, 4, "li"),
                  ("gaussian", 2, "none", 0, 1, "nn")]
SETS["stencil1"] = [("gaussian", 2, "stencil1", 0, 1, "nn"), ("sobel", 1, "stencil1", 0, 1, "nn"),
                    ("gaussian", 2, "none", 0, 1, "nn")]
SETS["all"] = SETS["row"] + SETS["col"] + SETS["checker"]

CHILD = r'''
import json, sys, torch
sys.path.insert(0, ROOT)
import paper_conf_cgo_maiercj18_b200 as kp, synth
vs = json.loads(sys.argv[1])
KEYS = json.loads(sys.argv[2]) if len(sys.argv) > 2 else {}
out = {}
bufs = {}
def buf(app, shape=None):
    if shape:
        W, H, B = shape; dt = torch.float32
    elif app == "median":
        W = H = 8192; B = 4; dt = torch.uint8
    elif app == "gauss_sobel":
        W, H, B, dt = 3840, 2160, 16, torch.float32
    else:
        W = H = 4096; B = 8; dt = torch.float32
    k = (W, H, B, dt)
    if k not in bufs:
        x = torch.empty((B, H, W), device="cuda", dtype=dt)
        synth.image_device("natural", 0x5EED0011, W, H, B, x.data_ptr(), dt == torch.uint8)
        bufs[k] = (x, torch.empty_like(x))
    return (W, H, B) + bufs[k]
for v in vs:
    app, r, sch, num, den, rc = v[:6]
    if app == "hotspot":  # 16384^2, 20 steps per call
        W = H = 16384
        if "hs" not in bufs:
            T = torch.empty((H, W), device="cuda"); P = torch.empty_like(T)
            synth.hotspot_device(0x5EED0030, W, H, T.data_ptr(), P.data_ptr())
            bufs["hs"] = (T, P, torch.empty_like(T))
        T, P, O = bufs["hs"]
        with kp.Plan(app, W, H, 1, sch, (num, den), rc, iters=20, **KEYS) as p:
            p.hotspot(T, P, O)
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for _ in range(3): p.hotspot(T, P, O)
            e1.record(); e1.synchronize()
            out["/".join(map(str, v))] = e0.elapsed_time(e1) / 3 / 20
        continue
    W, H, B, x, y = buf(app, v[6:] or None)
    with kp.Plan(app, W, H, r, sch, (num, den), rc, batch=B, **KEYS) as p:
        for _ in range(3): p.run(x, y)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for _ in range(20): p.run(x, y)
        e1.record(); e1.synchronize()
        out["/".join(map(str, v))] = e0.elapsed_time(e1) / 20
print("AB" + json.dumps(out))
'''.replace("ROOT", repr(ROOT))


def main():
    args = sys.argv[1:]
    sel = "row"
    if args and args[0] == "--set":
        sel, args = args[1], args[2:]
    rounds = int(os.environ.get("AB_ROUNDS", "3"))
    vs = SETS[sel]
    res = {lib: [] for lib in args}
    for _ in range(rounds):
        for lib in args:
            path, _, keys = lib.partition("@")  # lib.so@{"ring": 8}: plan keys for this arm only
            env = dict(os.environ, KPERF_LIB=os.path.abspath(path))
            o = subprocess.run([sys.executable, "-c", CHILD, json.dumps(vs), keys or os.environ.get("AB_KEYS", "{}")], env=env,
                               capture_output=True, text=True)
            line = [ln for ln in o.stdout.splitlines() if ln.startswith("AB")]
            if not line:
                print(lib, "FAILED", o.stderr[-2000:])
                res[lib].append({})
                continue
            res[lib].append(json.loads(line[0][2:]))
    keys = ["/".join(map(str, v)) for v in vs]
    print("variant".ljust(30) + "".join(os.path.basename(l.partition("@")[0])[:12].rjust(14)
                                        + l.partition("@")[2][:12].ljust(12) for l in args))
    for k in keys:
        row = k.ljust(30)
        for lib in args:
            xs = sorted(r[k] for r in res[lib] if k in r)
            row += (f"{xs[len(xs) // 2] * 1000:10.1f} us" if xs else "      fail").rjust(26)
        print(row)


if __name__ == "__main__":
    main()
