"""Multi-rank host logic of the sharded Hotspot on CPU (gloo, world size 2 and 3).

Each rank owns the row band kp.band_cuts(H, n)[rank:rank+2] with halo_rows =
perf_plan_get(plan, "halo_rows") rows on each side (queried from libkperf,
no GPU needed) and, every step, exchanges halos with the same choreography as
kperf.cu's NCCL path (my first halo rows -> rank-1's bottom halo, my last halo
rows -> rank+1's top halo), then advances its window one launch (1 step, or
TBLOCK steps under temporal blocking) with the
oracle's windowed Hotspot (global-coordinate mask).  The gathered bands must
equal the whole-grid oracle bit for bit: this pins the band partition, the
halo size and the exchange pattern the GPU path uses.
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
import paper_conf_cgo_maiercj18_b200 as kp
import synth

W, H, ITERS = 48, 61, 7


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _worker(rank, n, port, scheme, rate, recon, q, tb=1):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=n)
    try:
        cuts = kp.band_cuts(H, n)
        y0, y1 = cuts[rank], cuts[rank + 1]
        h = y1 - y0
        plan = kp.perf_plan("hotspot", W, h, 1, scheme, rate, recon)
        kp.perf_plan_set(plan, "global_h", H)
        kp.perf_plan_set(plan, "band_y0", y0)
        kp.perf_plan_set(plan, "tblock", tb)
        hb = kp.perf_plan_get(plan, "halo_rows")
        kp.perf_destroy(plan)
        T0, P = synth.hotspot(synth.SEED_C4, W, H)
        # band buffer rows [y0 - hb, y1 + hb); rows outside the grid are absent
        lo, hi = max(0, y0 - hb), min(H, y1 + hb)
        T = np.ascontiguousarray(T0[lo:hi].astype(np.float64))
        Pw = np.ascontiguousarray(P[lo:hi])
        prm = oracle.params("hotspot", W, H, 1, scheme, rate, recon, 8, tblock=tb)
        top = y0 - lo  # rows of top halo present
        for i in range(0, ITERS, tb):
            reqs = []
            if rank > 0:  # my first hb rows up, its last hb rows into my top halo
                reqs.append(dist.isend(torch.from_numpy(T[top:top + hb].copy()), rank - 1))
                buf_top = torch.empty((hb, W), dtype=torch.float64)
                reqs.append(dist.irecv(buf_top, rank - 1))
            if rank < n - 1:
                reqs.append(dist.isend(torch.from_numpy(T[top + h - hb:top + h].copy()), rank + 1))
                buf_bot = torch.empty((hb, W), dtype=torch.float64)
                reqs.append(dist.irecv(buf_bot, rank + 1))
            for r in reqs:
                r.wait()
            if rank > 0:
                T[:top] = buf_top.numpy()[hb - top:]
            if rank < n - 1:
                T[top + h:] = buf_bot.numpy()[:hi - y1]
            oracle.hotspot_window(prm, T, Pw, 0, lo, min(tb, ITERS - i))
        hmax = max(cuts[r + 1] - cuts[r] for r in range(n))  # gloo gathers equal shapes
        mine = torch.zeros((hmax, W), dtype=torch.float64)
        mine[:h] = torch.from_numpy(np.ascontiguousarray(T[top:top + h]))
        parts = [torch.empty((hmax, W), dtype=torch.float64) for r in range(n)]
        if rank == 0:
            dist.gather(mine, parts, dst=0)
            q.put(np.concatenate([parts[r].numpy()[:cuts[r + 1] - cuts[r]] for r in range(n)]))
        else:
            dist.gather(mine, None, dst=0)
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("n", [2, 3])
@pytest.mark.parametrize("scheme,rate,recon,tb", [("none", (0, 1), "nn", 1), ("row", (1, 2), "li", 1),
                                                  ("row", (3, 4), "nn", 1), ("checker", (1, 4), "li", 1),
                                                  ("col", (1, 2), "li", 1), ("row", (1, 2), "li", 3),
                                                  ("none", (0, 1), "nn", 4)])
def test_banded_hotspot_equals_whole_grid(n, scheme, rate, recon, tb):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, n, port, scheme, rate, recon, q, tb)) for r in range(n)]
    for p in procs:
        p.start()
    got = q.get(timeout=120)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    T0, P = synth.hotspot(synth.SEED_C4, W, H)
    want = oracle.hotspot(oracle.params("hotspot", W, H, 1, scheme, rate, recon, 8, tblock=tb), T0, P, ITERS)
    assert np.array_equal(got, want)


def test_band_cuts_and_halo():
    assert kp.band_cuts(16384, 8) == [2048 * k for k in range(9)]
    assert kp.band_cuts(10, 3) == [0, 3, 6, 10]
    with pytest.raises(ValueError):
        kp.band_cuts(2, 3)
    for scheme, rate, want in [("none", (0, 1), 1), ("row", (1, 2), 3), ("row", (3, 4), 5),
                               ("checker", (1, 8), 9), ("col", (1, 2), 1)]:
        h = kp.perf_plan("hotspot", 64, 64, 1, scheme, rate, "li")
        assert kp.perf_plan_get(h, "halo_rows") == want
        kp.perf_plan_set(h, "tblock", 4)  # a launch of 4 steps reads 4 rows further
        assert kp.perf_plan_get(h, "halo_rows") == want + 3
        kp.perf_destroy(h)
