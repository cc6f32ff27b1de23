"""Launch the temporally blocked Hotspot kernel for ncu captures: for each of
(row 1/2 LI, exact) two perf_run_hotspot calls of one launch each (tblock =
iters); with ncu -k regex:hotspot_tb the 2nd launch is the row kernel, the
4th the exact one.   usage: ncu_hotspot_tb.py [tblock] [N]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
import synth  # noqa: E402

tb = int(sys.argv[1]) if len(sys.argv) > 1 else 8
N = int(sys.argv[2]) if len(sys.argv) > 2 else 8192
T = torch.empty((N, N), device="cuda")
P = torch.empty_like(T)
o = torch.empty_like(T)
synth.hotspot_device(synth.SEED_C4, N, N, T.data_ptr(), P.data_ptr())
for sch, rt, rc in (("row", (1, 2), "li"), ("none", (0, 1), "nn")):
    with kp.Plan("hotspot", N, N, 1, sch, rt, rc, iters=tb, tblock=tb) as p:
        p.hotspot(T, P, o)
        p.hotspot(T, P, o)
torch.cuda.synchronize()
