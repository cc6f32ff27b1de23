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


def _exchange(buf, hp, dtype=torch.float64):
    """one halo exchange of a band buffer, rows exactly as libkperf's
    perf_band_halo says (the bookkeeping band_exchange_nccl uses)"""
    hb = hp["halo_rows"]
    reqs, recvs = [], []
    for nb, send, recv in ((hp["up_rank"], hp["send_up_row"], hp["recv_up_row"]),
                           (hp["down_rank"], hp["send_down_row"], hp["recv_down_row"])):
        if nb < 0:
            continue
        reqs.append(dist.isend(torch.from_numpy(np.ascontiguousarray(buf[send:send + hb])).to(dtype), nb))
        t = torch.empty((hb,) + buf.shape[1:], dtype=dtype)
        reqs.append(dist.irecv(t, nb))
        recvs.append((recv, t))
    for r in reqs:
        r.wait()
    for row, t in recvs:
        buf[row:row + hb] = t.numpy()


def _worker(rank, n, port, scheme, rate, recon, q, tb=1):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=n)
    try:
        cuts = kp.band_cuts(H, n)
        y0, y1 = cuts[rank], cuts[rank + 1]
        h = y1 - y0
        with kp.Plan("hotspot", W, h, 1, scheme, rate, recon, global_h=H, band_y0=y0, tblock=tb) as pl:
            hp = kp.perf_band_halo(pl.handle, rank, n)
            assert hp["halo_rows"] == pl.get("halo_rows")
        hb = hp["halo_rows"]
        T0, P = synth.hotspot(synth.SEED_C4, W, H)
        # band buffer rows [y0 - hb, y1 + hb) (perf_band_halo layout); rows outside the grid stay NaN
        T = np.full((hp["buf_rows"], W), np.nan)
        T[hb:hb + h] = T0[y0:y1]
        lo, hi = max(0, y0 - hb), min(H, y1 + hb)  # grid rows the buffer can hold
        Pw = np.ascontiguousarray(P[lo:hi])  # static power: the band's rows + halo, exchanged once on the GPU
        prm = oracle.params("hotspot", W, H, 1, scheme, rate, recon, 8, tblock=tb)
        a, b = lo - (y0 - hb), hi - (y0 - hb)  # buffer rows inside the grid
        for i in range(0, ITERS, tb):
            _exchange(T, hp)
            win = np.ascontiguousarray(T[a:b])
            oracle.hotspot_window(prm, win, Pw, 0, lo, min(tb, ITERS - i))
            T[a:b] = win
        hmax = max(cuts[r + 1] - cuts[r] for r in range(n))  # gloo gathers equal shapes
        mine = torch.zeros((hmax, W), dtype=torch.float64)
        mine[:h] = torch.from_numpy(np.ascontiguousarray(T[hb:hb + h]))
        parts = [torch.empty((hmax, W), dtype=torch.float64) for r in range(n)]
        if rank == 0:
            dist.gather(mine, parts, dst=0)
            q.put(np.concatenate([parts[r].numpy()[:cuts[r + 1] - cuts[r]] for r in range(n)]))
        else:
            dist.gather(mine, None, dst=0)
    finally:
        dist.destroy_process_group()


BW, BH = 96, 70  # one-shot band images


def _band_worker(rank, n, port, app, r, scheme, rate, recon, q):
    """C2/C3-style one-shot row bands (perf_run_band's layout): each rank holds
    only its own rows, fills the halo by one exchange, and evaluates its rows
    with the oracle on an image that is NaN everywhere outside its buffer --
    a missing halo row would poison the result.  Then the error metric of the
    sharded image: per-rank partial sums, all-reduced, finished by libkperf's
    perf_error_finish (the bookkeeping of perf_error_allreduce)."""
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=n)
    try:
        cuts = kp.band_cuts(BH, n)
        y0, y1 = cuts[rank], cuts[rank + 1]
        h = y1 - y0
        with kp.Plan(app, BW, h, r, scheme, rate, recon, global_h=BH, band_y0=y0, granule_bytes=32) as pl:
            hp = kp.perf_band_halo(pl.handle, rank, n)
            metric = pl.get("metric")
            hb = hp["halo_rows"]
            img = synth.image("natural", 0x5EED2200, BW, BH)
            buf = np.full((hp["buf_rows"], BW), np.nan)
            buf[hb:hb + h] = img[y0:y1]
            _exchange(buf, hp)
            view = np.full((BH, BW), np.nan, dtype=np.float32)
            lo, hi = max(0, y0 - hb), min(BH, y1 + hb)
            view[lo:hi] = buf[lo - (y0 - hb):hi - (y0 - hb)]
            xs, ys = np.meshgrid(np.arange(BW), np.arange(y0, y1))
            prm = oracle.params(app, BW, BH, r, scheme, rate, recon, 8)
            got = oracle.run_pixels(prm, view, xs.ravel(), ys.ravel()).reshape(h, BW)
            want = oracle.run(prm, img)[y0:y1]
            assert np.array_equal(got, want), "band rows differ from the whole image's"
            # sharded error: the plain definition per shard, summed over ranks
            ex = oracle.run(oracle.params(app, BW, BH, r), img)[y0:y1].astype(np.float32).astype(np.float64)
            ap = got.astype(np.float32).astype(np.float64)
            d = np.abs(ex - ap)
            name = {0: "mre", 1: "me", 2: "mae"}[metric]
            if name == "mre":
                nz = ex != 0
                sums = torch.tensor([np.sum(d[nz] / np.abs(ex[nz])), 0.0, float(nz.sum())], dtype=torch.float64)
            else:
                sums = torch.tensor([d.sum(), np.abs(ex).sum(), float(d.size)], dtype=torch.float64)
            dist.all_reduce(sums)
            v, c = kp.perf_error_finish(pl.handle, sums.tolist())
        if rank == 0:
            ex_all = oracle.run(oracle.params(app, BW, BH, r), img).astype(np.float32)
            ap_all = oracle.run(prm, img).astype(np.float32)
            q.put((v, c) + oracle.error(name, ex_all, ap_all))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("n", [3])
@pytest.mark.parametrize("app,r,scheme,rate,recon", [("gaussian", 2, "row", (1, 2), "li"),
                                                     ("sobel", 1, "checker", (3, 4), "nn"),
                                                     ("gauss_sobel", 2, "row", (3, 4), "li"),
                                                     ("gaussian", 1, "col", (1, 4), "li"),
                                                     ("sobel", 2, "none", (0, 1), "nn")])
def test_oneshot_bands_and_sharded_error(n, app, r, scheme, rate, recon):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_band_worker, args=(k, n, port, app, r, scheme, rate, recon, q)) for k in range(n)]
    for p in procs:
        p.start()
    v, c, ov, oc = q.get(timeout=120)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    assert c == oc and abs(v - ov) <= 1e-12 * max(1.0, ov)


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
