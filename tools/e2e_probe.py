"""PCIe ceiling for bench.py's e2e leg: pinned H2D alone, D2H alone, both at
once on two streams, and perf_run_host (C2 frame, 4096^2 fp32), CUDA events.
usage: e2e_probe.py"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402

W = H = 4096
nb = W * H * 4
hin = torch.rand((H, W)).pin_memory()
hout = torch.empty_like(hin).pin_memory()
d0 = torch.empty((H, W), device="cuda")
d1 = torch.empty((H, W), device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def timed(f, reps=10):
    f()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        f()
    e1.record()
    e1.synchronize()
    return e0.elapsed_time(e1) / reps


def both():
    ev = torch.cuda.Event()
    ev.record()
    s1.wait_event(ev)
    s2.wait_event(ev)
    with torch.cuda.stream(s1):
        d0.copy_(hin, non_blocking=True)
    with torch.cuda.stream(s2):
        hout.copy_(d1, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)
    torch.cuda.current_stream().wait_stream(s2)


print(f"H2D alone   {timed(lambda: d0.copy_(hin, non_blocking=True)):.3f} ms  ({nb / 1e6:.0f} MB)")
print(f"D2H alone   {timed(lambda: hout.copy_(d1, non_blocking=True)):.3f} ms")
print(f"H2D || D2H  {timed(both):.3f} ms")
st = torch.cuda.current_stream()
plan = kp.Plan("gaussian", W, H, 2, "row", (1, 2), "li", batch=1)
print(f"run_host    {timed(lambda: plan.run_host(hin, hout, st)):.3f} ms (row 1/2 LI, pipelined chunks)")
plan.close()


def chunked(nc, dep=True):
    """nc chunks: H2D on s1; D2H of chunk i on s2 after H2D of chunk i (no kernels)."""
    per = H // nc
    ev0 = torch.cuda.Event()
    ev0.record()
    s1.wait_event(ev0)
    s2.wait_event(ev0)
    evs = []
    for i in range(nc):
        with torch.cuda.stream(s1):
            d0[i * per:(i + 1) * per].copy_(hin[i * per:(i + 1) * per], non_blocking=True)
            e = torch.cuda.Event()
            e.record()
            evs.append(e)
    for i in range(nc):
        with torch.cuda.stream(s2):
            if dep:
                s2.wait_event(evs[i])
            hout[i * per:(i + 1) * per].copy_(d1[i * per:(i + 1) * per], non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)
    torch.cuda.current_stream().wait_stream(s2)


for nc in (1, 4, 16):
    print(f"chunks {nc:2d}: H2D || D2H, D2H(i) after H2D(i) {timed(lambda: chunked(nc)):.3f} ms; "
          f"independent {timed(lambda: chunked(nc, False)):.3f} ms")
