import numpy as np, torch, sys
sys.path.insert(0, '.')
import paper_conf_cgo_maiercj18_b200 as kp, synth
for app, r in [("gaussian",2),("sobel",1),("median",1),("gauss_sobel",2),("inversion",0)]:
    u8 = app=="median"
    W, H = (2100, 70) if u8 else (600, 70)
    img = synth.image("natural", 1, W, H, np.uint8 if u8 else np.float32)
    x = torch.from_numpy(img).cuda(); y = torch.empty_like(x)
    for s, rate, rc, ld in [("none",(0,1),"nn",0),("row",(1,2),"li",0),("row",(3,4),"nn",3),("col",(1,4),"li",0),("col",(1,2),"nn",0),("col",(3,4),"nn",0),("checker",(1,2),"li",0),("checker",(3,4),"nn",3)]:
        with kp.Plan(app, W, H, r, s, rate, rc, loader=ld) as p:
            p.run(x, y); torch.cuda.synchronize()
# compact keep-one checkerboard slots (every warp on the fast path: W % 256 == 0)
img = synth.image("natural", 2, 1024, 70, np.float32)
x = torch.from_numpy(img).cuda(); y = torch.empty_like(x)
for app, r in [("gaussian", 2), ("sobel", 1)]:
    for rate, rc in [((3, 4), "li"), ((3, 4), "nn"), ((7, 8), "li"), ((1, 2), "nn")]:
        with kp.Plan(app, 1024, 70, r, "checker", rate, rc) as p:
            p.run(x, y); torch.cuda.synchronize()
T, P = synth.hotspot(3, 600, 70)
T = torch.from_numpy(T).cuda(); P = torch.from_numpy(P).cuda(); o = torch.empty_like(T)
with kp.Plan("hotspot", 600, 70, 1, "row", (1,2), "li", iters=3) as p:
    p.hotspot(T, P, o); torch.cuda.synchronize()
# one-shot row bands (perf_run_band, halos filled by the caller) and the overlapped / graph-captured banded Hotspot
img = synth.image("natural", 3, 600, 120, np.float32)
x = torch.from_numpy(img).cuda()
for k, (y0, h) in enumerate([(0, 50), (50, 70)]):
    with kp.Plan("gaussian", 600, h, 2, "row", (1, 2), "li", global_h=120, band_y0=y0) as p:
        hp = kp.perf_band_halo(p.handle, k, 2)
        hb = hp["halo_rows"]
        buf = torch.zeros((hp["buf_rows"], 600), device="cuda")
        lo, hi = max(0, y0 - hb), min(120, y0 + h + hb)
        buf[lo - (y0 - hb):hi - (y0 - hb)] = x[lo:hi]
        out = torch.empty((h, 600), device="cuda")
        kp.perf_run_band(p.handle, buf, out); torch.cuda.synchronize()
T, P = synth.hotspot(4, 600, 120)
T = torch.from_numpy(T).cuda(); P = torch.from_numpy(P).cuda(); o = torch.empty_like(T)
plans = [kp.Plan("hotspot", 600, 60, 1, "row", (1, 2), "li", iters=3, global_h=120, band_y0=60 * b) for b in range(2)]
kp.perf_run_hotspot_bands_local([q.handle for q in plans], T, P, o); torch.cuda.synchronize()
print("sanitizer workload done")
