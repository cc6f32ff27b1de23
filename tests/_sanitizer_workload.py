import numpy as np, torch, sys
sys.path.insert(0, '.')
import paper_conf_cgo_maiercj18_b200 as kp, synth
for app, r in [("gaussian",2),("sobel",1),("median",1),("gauss_sobel",2),("inversion",0)]:
    u8 = app=="median"
    W, H = (2100, 70) if u8 else (600, 70)
    img = synth.image("natural", 1, W, H, np.uint8 if u8 else np.float32)
    x = torch.from_numpy(img).cuda(); y = torch.empty_like(x)
    for s, rate, rc, ld in [("none",(0,1),"nn",0),("row",(1,2),"li",0),("row",(3,4),"nn",3),("col",(1,4),"li",0),("checker",(1,2),"li",0),("checker",(3,4),"nn",3)]:
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
print("sanitizer workload done")
