"""SURVEY 8(e) on the GPU: one-shot row bands (perf_run_band), the sharded
error (perf_error_sums / perf_error_allreduce), the captured Hotspot loop
(PERF_KEY_GRAPH) -- on one device -- and, when the box has >= 2 GPUs, the
real NCCL paths (banded Hotspot with overlapped halo exchange, one-shot bands
with the NCCL halo fill, allreduced error) against the single-GPU results.

Row bands are defined on global rows (R2: the mask is anchored to
the image, not the band), so every comparison here is bit for bit.
"""
import os
import socket

import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    torch.cuda.init()


def _band_input(whole, y0, h, hp):
    """the band buffer perf_run_band reads (perf_band_halo layout), halo rows
    filled from the whole image as the exchange would; rows outside the image
    are NaN / 0xAB (never read)"""
    B, H, W = whole.shape
    hb = hp["halo_rows"]
    fill = float("nan") if whole.dtype == torch.float32 else 0xAB
    buf = torch.full((B, hp["buf_rows"], W), fill, dtype=whole.dtype, device=whole.device)
    lo, hi = max(0, y0 - hb), min(H, y0 + h + hb)
    buf[:, lo - (y0 - hb):hi - (y0 - hb)] = whole[:, lo:hi]
    return buf


@pytest.mark.parametrize("app,r,scheme,rate,recon", [
    ("gaussian", 2, "row", (1, 2), "li"), ("gaussian", 2, "row", (3, 4), "nn"), ("sobel", 1, "checker", (3, 4), "li"),
    ("sobel", 1, "col", (1, 2), "nn"), ("gauss_sobel", 2, "row", (1, 2), "li"), ("median", 1, "col", (1, 2), "nn"),
    ("median", 1, "row", (1, 4), "li"), ("gaussian", 1, "none", (0, 1), "nn"), ("inversion", 0, "row", (1, 2), "li"),
    ("gaussian", 2, "stencil1", (0, 1), "nn")])
@pytest.mark.parametrize("nb", [2, 3])
def test_oneshot_bands_equal_whole_image(app, r, scheme, rate, recon, nb):
    """C2/C3 sharded by rows: each band's output == the whole image's rows"""
    u8 = app == "median"
    W, H, B = 2100, 300, 2
    imgs = np.stack([synth.image("natural", 0x5EED2300 + b, W, H, np.uint8 if u8 else np.float32) for b in range(B)])
    x = torch.from_numpy(imgs).cuda()
    whole = torch.empty_like(x)
    keys = dict(tile1_w=16, tile1_h=16) if scheme == "stencil1" else {}
    with kp.Plan(app, W, H, r, scheme, rate, recon, batch=B, **keys) as p:
        p.run(x, whole)
    cuts = [0, 96, 208, H] if nb == 3 else [0, 144, H]  # Stencil1: bands start on tile rows
    for k in range(nb):
        y0, h = cuts[k], cuts[k + 1] - cuts[k]
        with kp.Plan(app, W, h, r, scheme, rate, recon, batch=B, global_h=H, band_y0=y0, **keys) as p:
            hp = kp.perf_band_halo(p.handle, k, nb)
            buf = _band_input(x, y0, h, hp)
            out = torch.empty((B, h, W), dtype=x.dtype, device="cuda")
            kp.perf_run_band(p.handle, buf, out)
            torch.cuda.synchronize()
        assert torch.equal(out, whole[:, y0:y0 + h]), (k, y0, h)


def test_oneshot_band_sampled_against_oracle():
    """a middle band of a C2-sized image in the bench's batch == the oracle"""
    W, H, B, nb, k = 4096, 4096, 2, 4, 1
    x = torch.empty((B, H, W), device="cuda")
    synth.image_device("natural", 0x5EED0011, W, H, B, x.data_ptr(), False)
    cuts = kp.band_cuts(H, nb)
    y0, h = cuts[k], cuts[k + 1] - cuts[k]
    with kp.Plan("gaussian", W, h, 2, "row", (1, 2), "li", batch=B, global_h=H, band_y0=y0) as p:
        hp = kp.perf_band_halo(p.handle, k, nb)
        buf = _band_input(x, y0, h, hp)
        out = torch.empty((B, h, W), device="cuda")
        kp.perf_run_band(p.handle, buf, out)
    torch.cuda.synchronize()
    img = synth.image("natural", 0x5EED0011 + 1, W, H)
    prm = oracle.params("gaussian", W, H, 2, "row", (1, 2), "li")
    ys = np.r_[y0, y0 + 1, y0 + 2, y0 + h - 3, y0 + h - 2, y0 + h - 1]
    yy, xx = np.meshgrid(ys, np.arange(0, W, 7), indexing="ij")
    want = oracle.run_pixels(prm, img, xx.ravel(), yy.ravel())
    got = out[1].cpu().numpy()[yy.ravel() - y0, xx.ravel()]
    assert np.all(np.abs(got - want) <= 1e-5 * np.abs(want))


def test_error_sums_add_over_shards():
    """perf_error_sums of two halves add up to the whole batch's sums;
    perf_error_allreduce without a communicator == perf_error"""
    W, H, B = 1000, 300, 4
    imgs = np.stack([synth.image("natural", 60 + b, W, H) for b in range(B)])
    x = torch.from_numpy(imgs).cuda()
    ex, ap = torch.empty_like(x), torch.empty_like(x)
    for metric in ("mre", "me", "mae"):
        with kp.Plan("sobel", W, H, 1, batch=B) as pe, \
                kp.Plan("sobel", W, H, 1, "row", (1, 2), "li", batch=B, metric=kp.METRIC[metric]) as p, \
                kp.Plan("sobel", W, H, 1, "row", (1, 2), "li", batch=B // 2, metric=kp.METRIC[metric]) as ph:
            pe.run(x, ex)
            p.run(x, ap)
            whole = kp.perf_error_sums(p.handle, ex, ap)
            halves = [kp.perf_error_sums(ph.handle, ex[s], ap[s]) for s in (slice(0, 2), slice(2, 4))]
            assert whole[2] == halves[0][2] + halves[1][2]
            for i in range(2):
                assert abs(whole[i] - (halves[0][i] + halves[1][i])) <= 1e-12 * max(1.0, abs(whole[i]))
            v, c = kp.perf_error_finish(p.handle, [a + b for a, b in zip(*halves)])
            assert (v, c) == pytest.approx(p.error(ex, ap), rel=1e-12)
            assert kp.perf_error_allreduce(p.handle, ex, ap) == p.error(ex, ap)


@pytest.mark.parametrize("tb", [1, 4])
def test_hotspot_graph_equals_eager(tb):
    """the captured ITERS loop (default) == eager launches, bit for bit; a
    replay after new inputs and after perf_plan_set re-capture stay right"""
    W, H = 700, 300
    T, P = synth.hotspot(9, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    ref = torch.empty_like(Td)
    out = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=7, tblock=tb, graph=0) as pe, \
            kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=7, tblock=tb) as pg:
        assert pg.get("graph") == 1
        pe.hotspot(Td, Pd, ref)
        for _ in range(2):
            out.fill_(float("nan"))
            pg.hotspot(Td, Pd, out)
            torch.cuda.synchronize()
            assert torch.equal(out, ref)
        Td2 = Td + 1.0  # same buffers, new contents: the replay reads them
        pe.hotspot(Td2, Pd, ref)
        pg.hotspot(Td2, Pd, out)
        torch.cuda.synchronize()
        assert torch.equal(out, ref)
        pe.set("iters", 3)
        pg.set("iters", 3)
        pe.hotspot(Td, Pd, ref)
        pg.hotspot(Td, Pd, out)
        torch.cuda.synchronize()
        assert torch.equal(out, ref)
        assert pg.get("graph") == 1


# ---------------------------------------------------------------------------
# real NCCL over >= 2 GPUs (skipped on one-GPU boxes)
def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _nccl_worker(rank, n, uid_q, res_q):
    import torch as t
    import paper_conf_cgo_maiercj18_b200 as k2
    import synth as sy
    t.cuda.set_device(rank)
    if rank == 0:
        uid = k2.perf_comm_unique_id()
        for _ in range(n - 1):
            uid_q.put(uid)
    else:
        uid = uid_q.get(timeout=60)
    res = {}
    # banded Hotspot, overlapped NCCL halos, graph-captured loop
    W, H, iters = 1024, 512, 13
    cuts = k2.band_cuts(H, n)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    T, P = sy.hotspot(31, W, H)
    Td = t.from_numpy(np.ascontiguousarray(T[y0:y0 + h])).cuda()
    Pd = t.from_numpy(np.ascontiguousarray(P[y0:y0 + h])).cuda()
    for overlap, graph in ((1, 1), (0, 0)):
        out = t.empty_like(Td)
        with k2.Plan("hotspot", W, h, 1, "row", (1, 2), "li", iters=iters, global_h=H, band_y0=y0,
                     overlap=overlap, graph=graph) as p:
            k2.perf_comm_init(p.handle, uid, rank, n)
            for _ in range(2):
                p.hotspot(Td, Pd, out)
            t.cuda.synchronize()
            res[f"hotspot_{overlap}{graph}"] = out.cpu().numpy()
            res[f"graph_{overlap}{graph}"] = p.get("graph")
    # one-shot bands with the NCCL halo fill + the allreduced error
    BW, BH, B = 2048, 256, 2
    imgs = np.stack([sy.image("natural", 70 + b, BW, BH) for b in range(B)])
    cuts = k2.band_cuts(BH, n)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    with k2.Plan("gaussian", BW, h, 2, "row", (1, 2), "li", batch=B, global_h=BH, band_y0=y0) as p, \
            k2.Plan("gaussian", BW, h, 2, batch=B, global_h=BH, band_y0=y0) as pe:
        k2.perf_comm_init(p.handle, uid, rank, n)
        k2.perf_comm_init(pe.handle, uid, rank, n)
        hp = k2.perf_band_halo(p.handle, rank, n)
        hb = hp["halo_rows"]
        buf = t.full((B, hp["buf_rows"], BW), float("nan"), device="cuda")
        buf[:, hb:hb + h] = t.from_numpy(imgs[:, y0:y0 + h]).cuda()  # own rows only: halos arrive by NCCL
        out = t.empty((B, h, BW), device="cuda")
        ex = t.empty_like(out)
        k2.perf_run_band(p.handle, buf, out)
        hpe = k2.perf_band_halo(pe.handle, rank, n)
        bufe = t.full((B, hpe["buf_rows"], BW), float("nan"), device="cuda")
        bufe[:, hpe["halo_rows"]:hpe["halo_rows"] + h] = t.from_numpy(imgs[:, y0:y0 + h]).cuda()
        k2.perf_run_band(pe.handle, bufe, ex)
        t.cuda.synchronize()
        res["band"] = out.cpu().numpy()
        res["err"] = k2.perf_error_allreduce(p.handle, ex, out)
    res_q.put((rank, res))


@pytest.mark.skipif(not torch.cuda.is_available() or torch.cuda.device_count() < 2, reason="needs >= 2 GPUs")
def test_nccl_paths_equal_single_gpu():
    import torch.multiprocessing as mp
    n = min(torch.cuda.device_count(), 4)
    ctx = mp.get_context("spawn")
    uid_q, res_q = ctx.Queue(), ctx.Queue()
    procs = [ctx.Process(target=_nccl_worker, args=(k, n, uid_q, res_q)) for k in range(n)]
    for p in procs:
        p.start()
    res = dict(res_q.get(timeout=600) for _ in range(n))
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    # single-GPU references
    W, H, iters = 1024, 512, 13
    T, P = synth.hotspot(31, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    whole = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=iters) as p:
        p.hotspot(Td, Pd, whole)
    whole = whole.cpu().numpy()
    for key in ("hotspot_11", "hotspot_00"):
        assert np.array_equal(np.concatenate([res[k][key] for k in range(n)]), whole), key
    assert res[0]["graph_11"] == 1
    BW, BH, B = 2048, 256, 2
    imgs = np.stack([synth.image("natural", 70 + b, BW, BH) for b in range(B)])
    x = torch.from_numpy(imgs).cuda()
    y, ye = torch.empty_like(x), torch.empty_like(x)
    with kp.Plan("gaussian", BW, BH, 2, "row", (1, 2), "li", batch=B) as p, kp.Plan("gaussian", BW, BH, 2, batch=B) as pe:
        p.run(x, y)
        pe.run(x, ye)
        v, c = p.error(ye, y)
    assert np.array_equal(np.concatenate([res[k]["band"] for k in range(n)], axis=1), y.cpu().numpy())
    for k in range(n):
        assert res[k]["err"][1] == c and abs(res[k]["err"][0] - v) <= 1e-12 * v
