"""GPU <-> oracle parity through the C ABI.

fp32 apps: |gpu - oracle| <= RTOL*|oracle| + ATOL[app] per element, with
RTOL = 1e-5 (north_star) and ATOL only for Sobel's cancellation near zero
(1e-6 x the stencil's magnitude scale sum|w| * 255).  u8 (median): bit-exact.
Shapes span several CTA tiles (512 fp32 / 2048 u8 columns, 128 rows) and a
ragged tail; the full BASELINE sizes are checked on sampled pixels.
"""
import itertools

import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402

RTOL = 1e-5
ATOL = {("gaussian", 1): 0.0, ("gaussian", 2): 0.0, ("inversion", 0): 0.0, ("hotspot", 1): 0.0,
        ("sobel", 1): 8 * 255e-6, ("sobel", 2): 96 * 255e-6, ("gauss_sobel", 2): 8 * 255e-6}

VARIANTS = [("none", (0, 1), "nn")] + [(s, r, rc) for s in ("row", "col", "checker")
                                        for r in ((1, 2), (1, 4), (3, 4)) for rc in ("nn", "li")]
FLOAT_APPS = [("gaussian", 1), ("gaussian", 2), ("sobel", 1), ("sobel", 2), ("inversion", 0),
              ("gauss_sobel", 2)]


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    torch.cuda.init()


def gpu_run(app, r, img, scheme, rate, recon, G_bytes=32, batch=1, **keys):
    H, W = img.shape[-2:]
    dev = torch.from_numpy(np.ascontiguousarray(img)).cuda()
    out = torch.empty_like(dev)
    with kp.Plan(app, W, H, r, scheme, rate, recon, granule_bytes=G_bytes, batch=batch, **keys) as p:
        p.run(dev, out)
        torch.cuda.synchronize()
    return out.cpu().numpy()


def assert_close(app, r, got, want):
    if got.dtype == np.uint8:
        bad = np.argwhere(got != want)
        assert bad.size == 0, f"{len(bad)} mismatches, first at {bad[:5].tolist()}"
        return
    tol = RTOL * np.abs(want) + ATOL[(app, r)]
    err = np.abs(got.astype(np.float64) - want)
    bad = np.argwhere(err > tol)
    assert bad.size == 0, (f"{len(bad)} / {err.size} outside tol; first {bad[:5].tolist()} "
                           f"got {got[tuple(bad[0])]} want {want[tuple(bad[0])]}")


# ---------------------------------------------------------------------------
@pytest.mark.parametrize("app,r", FLOAT_APPS)
@pytest.mark.parametrize("scheme,rate,recon", VARIANTS)
def test_float_apps_parity(app, r, scheme, rate, recon):
    # 2 strips of 1024 columns (last one ragged), 3 segments (last one ragged)
    W, H = 1100, 300
    img = synth.image("natural", synth.SEED_C2 + 1, W, H)
    got = gpu_run(app, r, img, scheme, rate, recon)
    want = oracle.run(oracle.params(app, W, H, r, scheme, rate, recon, 8), img)
    assert_close(app, r, got, want)


@pytest.mark.parametrize("scheme,rate,recon", VARIANTS)
def test_median_parity(scheme, rate, recon):
    W, H = 4200, 140  # 3 strips of 2048 u8 columns, ragged
    img = synth.image("natural", synth.SEED_C3, W, H, np.uint8)
    got = gpu_run("median", 1, img, scheme, rate, recon)
    want = oracle.run(oracle.params("median", W, H, 1, scheme, rate, recon, 32), img)
    assert_close("median", 1, got, want)


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("sobel", 1), ("gauss_sobel", 2), ("median", 1)])
@pytest.mark.parametrize("shape", [(1, 1), (1, 7), (7, 1), (3, 5), (130, 2), (2, 130), (513, 129), (1027, 33)])
def test_ragged_and_tiny_shapes(app, r, shape):
    W, H = shape
    u8 = app == "median"
    img = synth.image("pattern", 17, W, H, np.uint8 if u8 else np.float32)
    G = 32 if u8 else 8
    for scheme, rate, recon in [("none", (0, 1), "nn"), ("row", (1, 2), "li"), ("col", (1, 4), "nn"),
                                ("checker", (1, 2), "li"), ("row", (3, 4), "nn")]:
        if scheme == "checker" and H < rate[1]:
            continue
        got = gpu_run(app, r, img, scheme, rate, recon)
        want = oracle.run(oracle.params(app, W, H, r, scheme, rate, recon, G), img)
        assert_close(app, r, got, want)


@pytest.mark.parametrize("gbytes", [4, 12, 16, 64, 128])
def test_granule_sizes(gbytes):
    """G not a multiple of the lane chunk (4 fp32) takes the generic rebuild path."""
    W, H = 1024, 64
    img = synth.image("natural", 5, W, H)
    for scheme, rate, recon in [("col", (1, 2), "li"), ("checker", (3, 4), "nn"), ("col", (7, 8), "li")]:
        got = gpu_run("gaussian", 2, img, scheme, rate, recon, G_bytes=gbytes)
        want = oracle.run(oracle.params("gaussian", W, H, 2, scheme, rate, recon, gbytes // 4), img)
        assert_close("gaussian", 2, got, want)


def test_default_granule_is_128_bytes():
    """default cell width = the measured DRAM fill granule: 32 fp32 / 128 u8 pixels"""
    W, H = 1536, 96
    img = synth.image("natural", 21, W, H)
    for scheme, rate, recon in [("col", (1, 2), "li"), ("checker", (1, 4), "nn"), ("col", (3, 4), "nn")]:
        with kp.Plan("gaussian", W, H, 2, scheme, rate, recon) as p:
            assert p.get("granule_bytes") == 128
            x = torch.from_numpy(img).cuda()
            y = torch.empty_like(x)
            p.run(x, y)
        want = oracle.run(oracle.params("gaussian", W, H, 2, scheme, rate, recon, 32), img)
        assert_close("gaussian", 2, y.cpu().numpy(), want)
    u = synth.image("natural", 22, 4096, 64, np.uint8)
    for scheme, rate in [("col", (1, 2)), ("checker", (1, 2))]:
        with kp.Plan("median", 4096, 64, 1, scheme, rate, "li") as p:
            x = torch.from_numpy(u).cuda()
            y = torch.empty_like(x)
            p.run(x, y)
        want = oracle.run(oracle.params("median", 4096, 64, 1, scheme, rate, "li", 128), u)
        assert_close("median", 1, y.cpu().numpy(), want)


@pytest.mark.parametrize("den", [2, 3, 5, 6, 7, 8])
def test_all_denominators(den):
    W, H = 600, 90
    img = synth.image("natural", 31, W, H)
    for scheme in ("row", "col", "checker"):
        for num in sorted({1, den - 1}):
            for recon in ("nn", "li"):
                got = gpu_run("sobel", 1, img, scheme, (num, den), recon)
                want = oracle.run(oracle.params("sobel", W, H, 1, scheme, (num, den), recon, 8), img)
                assert_close("sobel", 1, got, want)


# ---------------------------------------------------------------------------
# invariants of the CUDA path itself
def test_rate0_bit_identical_to_exact():
    W, H = 1030, 200
    img = synth.image("natural", 3, W, H)
    ex = gpu_run("gaussian", 2, img, "none", (0, 1), "nn")
    for s in ("row", "col", "checker"):
        assert np.array_equal(gpu_run("gaussian", 2, img, s, (0, 4), "li"), ex)


def test_loaders_and_tiles_give_identical_bits():
    W, H = 2048, 260
    img = synth.image("natural", 9, W, H)
    for scheme, rate, recon, loaders in [("row", (1, 2), "li", (1, 2, 3)), ("none", (0, 1), "nn", (1, 2, 3)),
                                         ("col", (1, 4), "nn", (2, 3)), ("checker", (3, 4), "li", (2, 3))]:
        ref = gpu_run("sobel", 2, img, scheme, rate, recon)
        for ld in loaders:
            for th in (1, 7, 128, 1000):
                got = gpu_run("sobel", 2, img, scheme, rate, recon, loader=ld, tile_h=th)
                assert np.array_equal(got, ref), (scheme, ld, th)


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("sobel", 1), ("gaussian", 1), ("gauss_sobel", 2)])
@pytest.mark.parametrize("den", [2, 3, 4, 8])
@pytest.mark.parametrize("gbytes", [32, 128])
@pytest.mark.parametrize("W", [2048, 512, 256])
def test_checker_keep_one_compact_slots(app, r, den, gbytes, W):
    """Keep-one checkerboard with W a multiple of the warp width: every warp on
    the fast path, so the ring slots hold only the row's kept cells (kperf.cu
    chk_compact; W 256 / 512: the 2-consumer-warp CTAs of narrow images).
    == the oracle, and bit-identical to the scalar loader (loader 3:
    full-width slots); the compact layout is asserted to be engaged."""
    H = 300  # 3 segments (last ragged); W 2048: 2 strips
    if W < 2048 and app == "gauss_sobel" and den == 8:
        pytest.skip("covered at W 2048")
    img = synth.image("natural", 41 + den, W, H)
    with kp.Plan(app, W, H, r, "checker", (den - 1, den), "li", granule_bytes=gbytes) as p:
        assert p.get("chk_compact") == 1
    for recon in ("nn", "li"):
        got = gpu_run(app, r, img, "checker", (den - 1, den), recon, G_bytes=gbytes)
        want = oracle.run(oracle.params(app, W, H, r, "checker", (den - 1, den), recon, gbytes // 4), img)
        assert_close(app, r, got, want)
        full = gpu_run(app, r, img, "checker", (den - 1, den), recon, G_bytes=gbytes, loader=3)
        assert np.array_equal(got, full), (den, recon)


@pytest.mark.parametrize("scheme,rate,recon", [("col", (1, 2), "li"), ("col", (1, 4), "nn"), ("col", (3, 4), "li"),
                                                ("checker", (1, 2), "nn"), ("checker", (1, 4), "li"),
                                                ("checker", (3, 4), "nn")])
def test_cell_run_loader_gives_identical_bits(scheme, rate, recon):
    """128-B cells: TMA bulk runs of kept cells (loader 4) == 16-B cp.async
    (2, the default) == scalar loads (3), bit for bit; and == the oracle."""
    W, H = 2200, 150  # 3 strips, ragged
    img = synth.image("natural", 23, W, H)
    ref = gpu_run("gaussian", 2, img, scheme, rate, recon, G_bytes=128, loader=2)
    for ld in (0, 3, 4):
        got = gpu_run("gaussian", 2, img, scheme, rate, recon, G_bytes=128, loader=ld)
        assert np.array_equal(got, ref), (scheme, rate, recon, ld)
    want = oracle.run(oracle.params("gaussian", W, H, 2, scheme, rate, recon, 32), img)
    assert_close("gaussian", 2, ref, want)


def test_inline_producer_gives_identical_bits():
    """PERF_KEY_PRODUCER 2 (inline producer in -DKPERF_IPROD=1 builds, ignored
    otherwise) never changes results."""
    W, H = 2048, 260
    img = synth.image("natural", 19, W, H)
    for scheme, rate, recon in [("row", (1, 2), "li"), ("none", (0, 1), "nn"), ("row", (3, 4), "nn"),
                                ("stencil1", (0, 1), "nn")]:
        ref = gpu_run("gaussian", 2, img, scheme, rate, recon)
        assert np.array_equal(gpu_run("gaussian", 2, img, scheme, rate, recon, producer=2), ref)


def test_constant_image_rebuilds_exactly():
    W, H = 700, 150
    img = np.full((H, W), 93.0, dtype=np.float32)
    for s, rate, rc in VARIANTS:
        assert np.all(gpu_run("gaussian", 2, img, s, rate, rc) == 93.0)
        assert np.all(gpu_run("sobel", 1, img, s, rate, rc) == 0.0)


def test_batch_frames():
    W, H, B = 520, 70, 3
    imgs = np.stack([synth.image("natural", 100 + b, W, H) for b in range(B)])
    got = gpu_run("gaussian", 2, imgs, "row", (1, 2), "li", batch=B)
    for b in range(B):
        want = oracle.run(oracle.params("gaussian", W, H, 2, "row", (1, 2), "li"), imgs[b])
        assert_close("gaussian", 2, got[b], want)


def test_run_host_equals_run():
    W, H = 640, 96
    img = synth.image("natural", 4, W, H)
    out = np.zeros_like(img)
    with kp.Plan("sobel", W, H, 1, "checker", (1, 2), "li", granule_bytes=32) as p:
        p.run_host(img, out)
    assert np.array_equal(out, gpu_run("sobel", 1, img, "checker", (1, 2), "li"))


@pytest.mark.parametrize("app,r,scheme,rate,recon,W,H,B", [
    ("gaussian", 2, "row", (1, 2), "li", 1024, 1030, 1),   # 16 row chunks, ragged last chunk
    ("sobel", 1, "checker", (1, 4), "li", 700, 517, 3),    # batch: chunks per frame
    ("median", 1, "col", (1, 2), "nn", 2100, 300, 2),
    ("gauss_sobel", 2, "row", (3, 4), "nn", 520, 70, 1),   # one chunk
])
def test_run_host_pinned_pipeline(app, r, scheme, rate, recon, W, H, B):
    """perf_run_host with pinned buffers (captured copy/compute pipeline) is
    bit-identical to perf_run; a second buffer pair re-captures; pageable too."""
    u8 = app == "median"
    imgs = np.stack([synth.image("natural", 40 + b, W, H, np.uint8 if u8 else np.float32) for b in range(B)])
    dev = torch.from_numpy(imgs).cuda()
    want = torch.empty_like(dev)
    with kp.Plan(app, W, H, r, scheme, rate, recon, batch=B) as p:
        p.run(dev, want)
        torch.cuda.synchronize()
        want = want.cpu().numpy()
        hin = torch.from_numpy(imgs).pin_memory()
        for _ in range(2):  # first call captures, second replays
            hout = torch.zeros_like(hin).pin_memory()
            p.run_host(hin, hout)
            assert np.array_equal(hout.numpy(), want)
        hin2 = torch.from_numpy(imgs[::-1].copy()).pin_memory()  # new buffers: re-capture
        hout2 = torch.zeros_like(hin2).pin_memory()
        p.run_host(hin2, hout2)
        assert np.array_equal(hout2.numpy(), want[::-1])
        pageable = np.zeros_like(imgs)
        p.run_host(imgs, pageable)
        assert np.array_equal(pageable, want)


@pytest.mark.parametrize("app,r,rate,recon,W,H", [
    ("gaussian", 2, (1, 2), "li", 1024, 1030),
    ("sobel", 1, (1, 4), "nn", 700, 517),
    ("gauss_sobel", 2, (3, 4), "li", 520, 70),
    ("median", 1, (1, 2), "nn", 2100, 300),
])
def test_run_host_skips_perforated_rows(app, r, rate, recon, W, H):
    """Row scheme through perf_run_host: only the kept rows cross PCIe
    (PERF_KEY_HOST_SKIP).  Skipped rows of the host input are poisoned (NaN /
    0xFF) -- the output equals perf_run on the clean image bit for bit, with
    and without the skip, so no skipped row is ever read (a1)."""
    u8 = app == "median"
    img = synth.image("natural", 61, W, H, np.uint8 if u8 else np.float32)
    dev = torch.from_numpy(img).cuda()
    want = torch.empty_like(dev)
    num, den = rate
    kept = [(y % den == 0) if num == den - 1 else (y % den != den - 1) for y in range(H)]
    bad = img.copy()
    for y in range(H):
        if not kept[y]:
            bad[y] = 255 if u8 else np.nan
    with kp.Plan(app, W, H, r, "row", rate, recon) as p:
        p.run(dev, want)
        torch.cuda.synchronize()
        want = want.cpu().numpy()
        hin = torch.from_numpy(bad).pin_memory()
        for skip in (1, 0):
            p.set("host_skip", skip)
            hout = torch.zeros_like(hin).pin_memory()
            p.run_host(hin, hout)
            assert np.array_equal(hout.numpy(), want), f"host_skip={skip}"
        assert p.get("h2d_bytes") == H * W * img.itemsize  # (host_skip 0 now)
        p.set("host_skip", 1)
        assert p.get("h2d_bytes") == sum(kept) * W * img.itemsize


@pytest.mark.parametrize("scheme,rate,recon", [("none", (0, 1), "nn"), ("row", (1, 2), "li"), ("row", (3, 4), "nn"),
                                                ("col", (1, 2), "li"), ("checker", (3, 4), "nn")])
def test_gauss_sobel_three_warp_ctas(scheme, rate, recon):
    """The fused pipeline on whole 768- but not 1024-column strips (C5's 3840)
    runs CTAs of 3 consumer warps (kperf.cu make_params): W = 1536 (two
    strips), ragged segments, against the oracle."""
    W, H = 1536, 150
    img = synth.image("natural", 71, W, H)
    got = gpu_run("gauss_sobel", 2, img, scheme, rate, recon, G_bytes=128)
    want = oracle.run(oracle.params("gauss_sobel", W, H, 2, scheme, rate, recon, granule=32), img)
    assert_close("gauss_sobel", 2, got, want)


def test_device_generator_matches_host():
    for cls in ("flat", "natural", "pattern"):
        d = torch.empty((2, 300, 500), dtype=torch.float32, device="cuda")
        synth.image_device(cls, 77, 500, 300, 2, d.data_ptr(), False)
        u = torch.empty((300, 500), dtype=torch.uint8, device="cuda")
        synth.image_device(cls, 77, 500, 300, 1, u.data_ptr(), True)
        torch.cuda.synchronize()
        assert np.array_equal(d[0].cpu().numpy(), synth.image(cls, 77, 500, 300))
        assert np.array_equal(d[1].cpu().numpy(), synth.image(cls, 78, 500, 300))
        assert np.array_equal(u.cpu().numpy(), synth.image(cls, 77, 500, 300, np.uint8))
    T = torch.empty((64, 96), device="cuda")
    P = torch.empty((64, 96), device="cuda")
    synth.hotspot_device(5, 96, 64, T.data_ptr(), P.data_ptr())
    torch.cuda.synchronize()
    Th, Ph = synth.hotspot(5, 96, 64)
    assert np.array_equal(T.cpu().numpy(), Th) and np.array_equal(P.cpu().numpy(), Ph)


# ---------------------------------------------------------------------------
# error metric (a5)
@pytest.mark.parametrize("app,r,metric", [("gaussian", 2, "mre"), ("sobel", 1, "me"), ("median", 1, "mre"),
                                          ("gaussian", 2, "mae")])
def test_error_metric(app, r, metric):
    W, H = 1500, 333
    u8 = app == "median"
    img = synth.image("natural", 12, W, H, np.uint8 if u8 else np.float32)
    ex = gpu_run(app, r, img, "none", (0, 1), "nn")
    ap = gpu_run(app, r, img, "row", (1, 2), "li")
    with kp.Plan(app, W, H, r, "row", (1, 2), "li", metric=kp.METRIC[metric]) as p:
        v, c = p.error(torch.from_numpy(ex).cuda(), torch.from_numpy(ap).cuda())
    # same buffers through the oracle's metric
    ov, oc = oracle.error(metric, ex, ap)
    assert c == oc
    assert abs(v - ov) <= 1e-9 * max(1.0, abs(ov))
    # end to end: the oracle's own exact/perforated outputs (north_star: 1e-6)
    oe = oracle.run(oracle.params(app, W, H, r, "none", (0, 1), "nn", 32 if u8 else 8), img)
    oa = oracle.run(oracle.params(app, W, H, r, "row", (1, 2), "li", 32 if u8 else 8), img)
    assert abs(v - oracle.error(metric, oe, oa)[0]) <= 1e-6


# ---------------------------------------------------------------------------
# Hotspot (a6)
@pytest.mark.parametrize("scheme,rate,recon", [("none", (0, 1), "nn"), ("row", (1, 2), "nn"),
                                               ("row", (1, 2), "li"), ("row", (3, 4), "li"),
                                               ("col", (1, 2), "li"), ("checker", (1, 4), "nn")])
@pytest.mark.parametrize("iters", [1, 6])
def test_hotspot_parity(scheme, rate, recon, iters):
    W, H = 1100, 260
    T, P = synth.hotspot(synth.SEED_C4, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    out = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, scheme, rate, recon, iters=iters, granule_bytes=32) as p:
        p.hotspot(Td, Pd, out)
        torch.cuda.synchronize()
    want = oracle.hotspot(oracle.params("hotspot", W, H, 1, scheme, rate, recon, 8), T, P, iters)
    assert_close("hotspot", 1, out.cpu().numpy(), want)
    assert np.array_equal(Td.cpu().numpy(), T)  # temp_in untouched


@pytest.mark.parametrize("scheme,rate,recon", [("none", (0, 1), "nn"), ("row", (1, 2), "li"),
                                               ("row", (3, 4), "nn"), ("checker", (1, 2), "li")])
@pytest.mark.parametrize("nb", [2, 3, 4])
@pytest.mark.parametrize("tb", [1, 4])
@pytest.mark.parametrize("overlap,graph", [(1, 1), (0, 0), (1, 0)])
def test_hotspot_bands_equal_whole_grid(scheme, rate, recon, nb, tb, overlap, graph):
    """Sharding semantics: row bands with halo exchange == one grid, bit for bit
    (tb > 1: temporally blocked launches, one halo exchange per launch).
    overlap: boundary rows first, their exchange on a second stream while the
    interior computes; graph: the loop captured and replayed
    (two calls: capture, then replay)."""
    if tb > 1 and scheme == "checker":
        pytest.skip("temporal blocking: NONE / ROW schemes")
    W, H, iters = 640, 200, 9
    T, P = synth.hotspot(7, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    whole = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, scheme, rate, recon, iters=iters, tblock=tb) as p:
        p.hotspot(Td, Pd, whole)
    cuts = np.linspace(0, H, nb + 1).astype(int)
    cuts[1:-1] += 3  # uneven bands
    plans = []
    for b in range(nb):
        h = int(cuts[b + 1] - cuts[b])
        plans.append(kp.Plan("hotspot", W, h, 1, scheme, rate, recon, iters=iters, global_h=H,
                             band_y0=int(cuts[b]), tblock=tb, overlap=overlap, graph=graph))
    for _ in range(2):
        banded = torch.full_like(Td, float("nan"))
        kp.perf_run_hotspot_bands_local([q.handle for q in plans], Td, Pd, banded)
        torch.cuda.synchronize()
        assert torch.equal(banded, whole)
    assert plans[0].get("graph") == graph  # (2 would mean the capture failed)
    for q in plans:
        q.close()


@pytest.mark.parametrize("scheme,rate,recon,tb", [("none", (0, 1), "nn", 1), ("row", (1, 2), "li", 1),
                                                  ("row", (3, 4), "nn", 1), ("checker", (1, 2), "li", 1),
                                                  ("col", (1, 4), "nn", 1), ("row", (1, 2), "li", 4),
                                                  ("none", (0, 1), "nn", 8)])
@pytest.mark.parametrize("nb", [2, 3])
def test_hotspot_p2p_bands_equal_whole_grid(scheme, rate, recon, tb, nb):
    """NEXT-4 on one device: halo rows stored by the step kernels straight into
    the neighbours' band buffers + epoch flags == one grid, bit for bit."""
    W, H, iters = 640, 200, 9
    T, P = synth.hotspot(17, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    whole = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, scheme, rate, recon, iters=iters, tblock=tb) as p:
        p.hotspot(Td, Pd, whole)
    cuts = np.linspace(0, H, nb + 1).astype(int)
    cuts[1:-1] -= 5  # uneven bands
    plans = [kp.Plan("hotspot", W, int(cuts[b + 1] - cuts[b]), 1, scheme, rate, recon, iters=iters, global_h=H,
                     band_y0=int(cuts[b]), tblock=tb, p2p=1) for b in range(nb)]
    banded = torch.full_like(Td, float("nan"))
    for _ in range(2):  # twice: the epoch counters carry across calls
        kp.perf_run_hotspot_bands_local([q.handle for q in plans], Td, Pd, banded)
        torch.cuda.synchronize()
        assert torch.equal(banded, whole)
    for q in plans:
        q.close()


def _p2p_worker(rank, n, W, H, iters, tb, scheme, rate, recon, blobs, barrier, out_q):
    import torch as t
    import paper_conf_cgo_maiercj18_b200 as kp2
    import synth as sy
    t.cuda.set_device(0)
    cuts = kp2.band_cuts(H, n)
    y0, h = cuts[rank], cuts[rank + 1] - cuts[rank]
    T, P = sy.hotspot(23, W, H)
    Td = t.from_numpy(np.ascontiguousarray(T[y0:y0 + h])).cuda()
    Pd = t.from_numpy(np.ascontiguousarray(P[y0:y0 + h])).cuda()
    out = t.empty_like(Td)
    with kp2.Plan("hotspot", W, h, 1, scheme, rate, recon, iters=iters, global_h=H, band_y0=y0, tblock=tb) as p:
        blobs[rank] = kp2.perf_p2p_export(p.handle)
        barrier.wait(timeout=120)
        kp2.perf_p2p_attach(p.handle, blobs[rank - 1] if rank > 0 else None, blobs[rank + 1] if rank < n - 1 else None)
        barrier.wait(timeout=120)  # every rank attached before any rank runs
        p.hotspot(Td, Pd, out)
        t.cuda.synchronize()
        out_q.put((rank, out.cpu().numpy()))
        barrier.wait(timeout=300)  # the neighbours' buffers stay mapped until everyone is done


@pytest.mark.parametrize("scheme,rate,recon,tb", [("row", (1, 2), "li", 1), ("row", (1, 2), "li", 4)])
def test_hotspot_p2p_ipc_two_processes(scheme, rate, recon, tb):
    """NEXT-4 through real CUDA IPC: two processes (two contexts on this one
    GPU) run adjacent bands with perf_p2p_export / perf_p2p_attach; the halo
    stores and flags cross the process boundary.  == one grid, bit for bit."""
    import torch.multiprocessing as mp
    W, H, iters, n = 520, 96, 6, 2
    T, P = synth.hotspot(23, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    whole = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, scheme, rate, recon, iters=iters, tblock=tb) as p:
        p.hotspot(Td, Pd, whole)
    torch.cuda.synchronize()
    ctx = mp.get_context("spawn")
    mgr = ctx.Manager()
    blobs = mgr.dict()
    barrier = mgr.Barrier(n)
    out_q = ctx.Queue()
    procs = [ctx.Process(target=_p2p_worker, args=(r, n, W, H, iters, tb, scheme, rate, recon, blobs, barrier, out_q))
             for r in range(n)]
    for pr in procs:
        pr.start()
    parts = dict(out_q.get(timeout=300) for _ in range(n))
    for pr in procs:
        pr.join(timeout=120)
        assert pr.exitcode == 0
    got = np.concatenate([parts[r] for r in range(n)])
    assert np.array_equal(got, whole.cpu().numpy())


# ---------------------------------------------------------------------------
# Hotspot temporal blocking (R19): TBLOCK steps per
# launch, T perforated at the first step of each launch -- oracle `tblock`
@pytest.mark.parametrize("scheme,rate,recon", [("none", (0, 1), "nn"), ("row", (1, 2), "li"),
                                               ("row", (1, 2), "nn"), ("row", (3, 4), "li"),
                                               ("row", (1, 3), "nn"), ("row", (7, 8), "li")])
@pytest.mark.parametrize("tb,iters", [(2, 1), (2, 7), (4, 16), (8, 13), (3, 9)])
def test_hotspot_tblock_parity(scheme, rate, recon, tb, iters):
    W, H = 1100, 260  # several 144..156-column x 32..44-row tiles, ragged tails
    T, P = synth.hotspot(synth.SEED_C4, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    out = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, scheme, rate, recon, iters=iters, tblock=tb) as p:
        p.hotspot(Td, Pd, out)
        torch.cuda.synchronize()
    want = oracle.hotspot(oracle.params("hotspot", W, H, 1, scheme, rate, recon, 8, tblock=tb), T, P, iters)
    assert_close("hotspot", 1, out.cpu().numpy(), want)
    assert np.array_equal(Td.cpu().numpy(), T)


@pytest.mark.parametrize("shape", [(1, 1), (5, 3), (7, 2), (101, 13), (1101, 97), (160, 48), (144, 32)])
@pytest.mark.parametrize("tb", [2, 8])
def test_hotspot_tblock_ragged(shape, tb):
    W, H = shape  # W % 4 != 0 takes the scalar loader
    T, P = synth.hotspot(3, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    out = torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=11, tblock=tb) as p:
        p.hotspot(Td, Pd, out)
        torch.cuda.synchronize()
    want = oracle.hotspot(oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8, tblock=tb), T, P, 11)
    assert_close("hotspot", 1, out.cpu().numpy(), want)


def test_hotspot_tblock1_is_per_step():
    W, H = 300, 70
    T, P = synth.hotspot(9, W, H)
    Td, Pd = torch.from_numpy(T).cuda(), torch.from_numpy(P).cuda()
    a, b = torch.empty_like(Td), torch.empty_like(Td)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=5) as p:
        p.hotspot(Td, Pd, a)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=5, tblock=1) as p:
        p.hotspot(Td, Pd, b)
    torch.cuda.synchronize()
    assert torch.equal(a, b)
    with pytest.raises(RuntimeError):
        with kp.Plan("hotspot", W, H, 1, "col", (1, 2), "li", iters=5, tblock=2) as p:
            p.hotspot(Td, Pd, b)


def test_c4_hotspot_tblock_cone_sampled():
    """4096^2 x 40 steps with TBLOCK 4 (the bench's C4 temporal-blocking
    variant); oracle on the dependency cones of a few patches"""
    W = H = 4096
    iters, tb = 40, 4
    T = torch.empty((H, W), device="cuda")
    P = torch.empty((H, W), device="cuda")
    synth.hotspot_device(synth.SEED_C4, W, H, T.data_ptr(), P.data_ptr())
    out = torch.empty_like(T)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=iters, tblock=tb) as p:
        p.hotspot(T, P, out)
    torch.cuda.synchronize()
    Th, Ph = T.cpu().numpy(), P.cpu().numpy()
    o = out.cpu().numpy()
    prm = oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", tblock=tb)
    for x0, y0 in [(0, 0), (2000, 1500), (4090, 4090), (151, 39), (777, 4093)]:
        w = min(6, W - x0)
        h = min(3, H - y0)
        want = oracle.hotspot_rect(prm, Th, Ph, iters, x0, y0, w, h)
        assert_close("hotspot", 1, o[y0:y0 + h, x0:x0 + w], want)


# ---------------------------------------------------------------------------
# BASELINE sizes in the bench's launch configuration, sampled pixels
def _samples(W, H, n, seed):
    rng = np.random.default_rng(seed)
    xs = np.r_[0, W - 1, 0, W - 1, rng.integers(0, W, n)]
    ys = np.r_[0, 0, H - 1, H - 1, rng.integers(0, H, n)]
    return xs, ys


def test_c1_full_image():
    W = H = 512
    img = synth.image("natural", synth.SEED_C1, W, H)
    got = gpu_run("gaussian", 2, img, "row", (1, 2), "li")
    want = oracle.run(oracle.params("gaussian", W, H, 2, "row", (1, 2), "li"), img)
    assert_close("gaussian", 2, got, want)


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("sobel", 1)])
@pytest.mark.parametrize("scheme,rate,recon", [(s, r, rc) for s in ("row", "col", "checker")
                                               for r in ((1, 2), (1, 4)) for rc in ("nn", "li")])
def test_c2_sampled(app, r, scheme, rate, recon):
    W = H = 4096
    img = synth.image("natural", synth.SEED_C2 + 1, W, H)
    got = gpu_run(app, r, img, scheme, rate, recon)
    xs, ys = _samples(W, H, 400, 2)
    want = oracle.run_pixels(oracle.params(app, W, H, r, scheme, rate, recon, 8), img, xs, ys)
    assert_close(app, r, got[ys, xs], want)


def test_c3_sampled():
    W = H = 8192
    img = synth.image("natural", synth.SEED_C3, W, H, np.uint8)
    for rate in ((1, 2), (1, 4), (3, 4)):
        got = gpu_run("median", 1, img, "col", rate, "nn")
        xs, ys = _samples(W, H, 2000, 3)
        want = oracle.run_pixels(oracle.params("median", W, H, 1, "col", rate, "nn", 32), img, xs, ys)
        assert np.array_equal(got[ys, xs], want)


def test_c4_hotspot_cone_sampled():
    """4096^2 x 40 steps; oracle on the dependency cones of a few patches."""
    W = H = 4096
    iters = 40
    T = torch.empty((H, W), device="cuda")
    P = torch.empty((H, W), device="cuda")
    synth.hotspot_device(synth.SEED_C4, W, H, T.data_ptr(), P.data_ptr())
    out = torch.empty_like(T)
    with kp.Plan("hotspot", W, H, 1, "row", (1, 2), "li", iters=iters) as p:
        p.hotspot(T, P, out)
    torch.cuda.synchronize()
    Th, Ph = T.cpu().numpy(), P.cpu().numpy()
    o = out.cpu().numpy()
    prm = oracle.params("hotspot", W, H, 1, "row", (1, 2), "li")
    for x0, y0 in [(0, 0), (2000, 1500), (4090, 4090), (777, 4093)]:
        w = min(6, W - x0)
        h = min(3, H - y0)
        want = oracle.hotspot_rect(prm, Th, Ph, iters, x0, y0, w, h)
        assert_close("hotspot", 1, o[y0:y0 + h, x0:x0 + w], want)


def test_c5_frames_sampled():
    W, H, B = 3840, 2160, 4
    frames = torch.empty((B, H, W), device="cuda")
    synth.image_device("natural", synth.SEED_C5, W, H, B, frames.data_ptr(), False)
    out = torch.empty_like(frames)
    with kp.Plan("gauss_sobel", W, H, 2, "row", (1, 2), "li", batch=B) as p:
        p.run(frames, out)
    torch.cuda.synchronize()
    prm = oracle.params("gauss_sobel", W, H, 2, "row", (1, 2), "li")
    for b in (0, B - 1):
        img = synth.image("natural", synth.SEED_C5 + b, W, H)
        xs, ys = _samples(W, H, 300, 10 + b)
        want = oracle.run_pixels(prm, img, xs, ys)
        assert_close("gauss_sobel", 2, out[b].cpu().numpy()[ys, xs], want)


# ---------------------------------------------------------------------------
# NEXT-1: Stencil1 -- tile interior loaded, halo NN from the tile
@pytest.mark.parametrize("app,r", [("gaussian", 1), ("gaussian", 2), ("sobel", 1), ("sobel", 2), ("inversion", 0),
                                   ("median", 1)])
@pytest.mark.parametrize("tile", [(16, 16), (32, 8), (64, 4), (256, 1), (16, 5), (128, 33)])
def test_stencil1_parity(app, r, tile):
    u8 = app == "median"
    W, H = (4200, 140) if u8 else (1100, 300)
    img = synth.image("natural", 41, W, H, np.uint8 if u8 else np.float32)
    got = gpu_run(app, r, img, "stencil1", (0, 1), "nn", tile1_w=tile[0], tile1_h=tile[1])
    want = oracle.run(oracle.params(app, W, H, r, "stencil1", (0, 1), "nn", tile=tile), img)
    assert_close(app, r, got, want)


@pytest.mark.parametrize("shape", [(1, 1), (7, 3), (130, 2), (513, 129), (1027, 33)])
def test_stencil1_ragged(shape):
    W, H = shape
    img = synth.image("pattern", 43, W, H)
    for tile in [(16, 16), (32, 7)]:
        got = gpu_run("gaussian", 2, img, "stencil1", (0, 1), "nn", tile1_w=tile[0], tile1_h=tile[1])
        want = oracle.run(oracle.params("gaussian", W, H, 2, "stencil1", (0, 1), "nn", tile=tile), img)
        assert_close("gaussian", 2, got, want)


def test_stencil1_whole_image_tile_is_exact():
    W, H = 250, 100
    img = synth.image("natural", 44, W, H)
    ex = gpu_run("sobel", 1, img, "none", (0, 1), "nn")
    assert np.array_equal(gpu_run("sobel", 1, img, "stencil1", (0, 1), "nn", tile1_w=256, tile1_h=128), ex)


# ---------------------------------------------------------------------------
# NEXT-2: the paper's error orderings reproduced through the GPU path
def test_paper_orderings_on_gpu():
    """Sec. 6.3 and Fig. 7 (:790-800) on synthetic stand-ins"""
    W = H = 512
    def mre(app, r, img, scheme, rate, recon, **k):
        ex = gpu_run(app, r, img, "none", (0, 1), "nn")
        ap = gpu_run(app, r, img, scheme, rate, recon, **k)
        with kp.Plan(app, W, H, r) as p:
            return p.error(torch.from_numpy(ex).cuda(), torch.from_numpy(ap).cuda())[0]
    nat = synth.image("natural", 0x5EED3100, W, H)
    for app, r in (("gaussian", 1), ("inversion", 0)):
        r1n, r2n = mre(app, r, nat, "row", (1, 2), "nn"), mre(app, r, nat, "row", (3, 4), "nn")
        r1l = mre(app, r, nat, "row", (1, 2), "li")
        assert r2n > r1n > r1l and r1n < 0.04  # :822-833
    s1 = mre("gaussian", 1, nat, "stencil1", (0, 1), "nn")
    assert s1 < 0.01 and s1 < mre("gaussian", 1, nat, "row", (1, 2), "nn")  # :824-826, :833-834
    errs = [mre("median", 1, synth.image(c, 0x5EED3200, W, H, np.uint8), "row", (1, 2), "nn")
            for c in ("flat", "natural", "pattern")]
    assert errs[0] < errs[1] < errs[2]  # Fig. 7: 0.12% < 5.05% < 19.32%


@pytest.mark.parametrize("gbytes", [32, 64, 128, 256, 512])
@pytest.mark.parametrize("rate", [(1, 2), (1, 3), (2, 3), (1, 4), (3, 4), (1, 8), (7, 8)])
def test_median_col_nn_cell_lanes(gbytes, rate):
    """Median, column NN: cell-grouped lanes and the all-skipped-warp shortcut
    (kernel.cuh MEDC) -- bit-exact against the oracle's true median; two full
    2048-column strips + a ragged one (identity lanes), every den / num, cells
    of 2..32 lanes (including cells straddling warps' cell groups)"""
    W, H = 4096 + 333, 150
    img = synth.image("natural", 0x5EED2400 + gbytes, W, H, np.uint8)
    got = gpu_run("median", 1, img, "col", rate, "nn", G_bytes=gbytes)
    want = oracle.run(oracle.params("median", W, H, 1, "col", rate, "nn", gbytes), img)
    assert_close("median", 1, got, want)
    pat = synth.image("pattern", 0x5EED2500, W, H, np.uint8)  # high-frequency: every window differs
    got = gpu_run("median", 1, pat, "col", rate, "nn", G_bytes=gbytes, batch=1)
    assert_close("median", 1, got, oracle.run(oracle.params("median", W, H, 1, "col", rate, "nn", gbytes), pat))


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("sobel", 1), ("gauss_sobel", 2), ("inversion", 0)])
@pytest.mark.parametrize("scheme,rate", [("col", (1, 2)), ("col", (1, 4)), ("col", (3, 4)), ("col", (1, 8)),
                                         ("col", (7, 8)), ("checker", (1, 2)), ("checker", (3, 4)),
                                         ("checker", (7, 8))])
@pytest.mark.parametrize("gbytes", [32, 128])
def test_tma_cell_loads(app, r, scheme, rate, gbytes):
    """TMA tensor-tile cell loads (loader 5, the auto choice for fp32 column and
    keep-one checkerboard cells): bit-identical to the 16-B cp.async loader
    (loader 2, full-width / compact slots) and == the oracle; two 1024-column
    strips and a third, 3 row segments, batch 2"""
    W, H, B = 3072, 300, 2
    imgs = np.stack([synth.image("natural", 0x5EED2600 + b, W, H) for b in range(B)])
    for recon in ("nn", "li"):
        tma = gpu_run(app, r, imgs, scheme, rate, recon, G_bytes=gbytes, batch=B, loader=5)
        ref = gpu_run(app, r, imgs, scheme, rate, recon, G_bytes=gbytes, batch=B, loader=2)
        assert np.array_equal(tma, ref), (recon,)
        auto = gpu_run(app, r, imgs, scheme, rate, recon, G_bytes=gbytes, batch=B)
        assert np.array_equal(auto, ref)
    want = oracle.run(oracle.params(app, W, H, r, scheme, rate, "li", gbytes // 4), imgs[1])
    assert_close(app, r, tma[1], want)


def test_tma_loader_refuses_unsupported_shapes():
    """loader 5 on shapes the tensor-tile path does not cover: a clear error,
    and the auto loader silently keeps cp.async (results unchanged)"""
    img = synth.image("natural", 7, 1100, 64)
    for scheme, rate in (("col", (1, 2)), ("checker", (1, 4)), ("row", (1, 2))):
        with pytest.raises(kp.PerfError):
            gpu_run("gaussian", 2, img, scheme, rate, "li", loader=5)
    got = gpu_run("gaussian", 2, img, "col", (1, 2), "li", G_bytes=128)
    want = oracle.run(oracle.params("gaussian", 1100, 64, 2, "col", (1, 2), "li", 32), img)
    assert_close("gaussian", 2, got, want)


def test_tma_cell_loads_in_row_bands():
    """perf_run_band with TMA cell loads (the frame pitch of the band buffer is
    buf_rows): bands == the whole image"""
    W, H, B = 2048, 200, 2
    imgs = np.stack([synth.image("natural", 0x5EED2700 + b, W, H) for b in range(B)])
    x = torch.from_numpy(imgs).cuda()
    whole = torch.empty_like(x)
    for scheme, rate in (("col", (1, 2)), ("checker", (3, 4))):
        with kp.Plan("gaussian", W, H, 2, scheme, rate, "li", batch=B, loader=5) as p:
            p.run(x, whole)
        for k, (y0, h) in enumerate(((0, 90), (90, 110))):
            with kp.Plan("gaussian", W, h, 2, scheme, rate, "li", batch=B, global_h=H, band_y0=y0, loader=5) as p:
                hp = kp.perf_band_halo(p.handle, k, 2)
                hb = hp["halo_rows"]
                buf = torch.full((B, hp["buf_rows"], W), float("nan"), device="cuda")
                lo, hi = max(0, y0 - hb), min(H, y0 + h + hb)
                buf[:, lo - (y0 - hb):hi - (y0 - hb)] = x[:, lo:hi]
                out = torch.empty((B, h, W), device="cuda")
                kp.perf_run_band(p.handle, buf, out)
                torch.cuda.synchronize()
            assert torch.equal(out, whole[:, y0:y0 + h]), (scheme, k)


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("gaussian", 1), ("sobel", 1), ("sobel", 2), ("gauss_sobel", 2)])
@pytest.mark.parametrize("rate", [(1, 2), (3, 4)])
@pytest.mark.parametrize("recon", ["nn", "li"])
def test_folded_row_rebuild(app, r, rate, recon):
    """The row scheme's rebuild folded into the vertical pass (fold.cuh,
    PERF_KEY_FOLD, default on for interior segments): bit-identical to the
    per-row rebuild-then-filter path (PERF_KEY_FOLD 0) on integer-valued
    images, and == the oracle.  2 frames of 2048 x 600: 5 row segments per
    frame, the first and last (image borders) on the per-row path; a ragged
    tile_h run and a banded run too."""
    W, H, B = 2048, 600, 2
    imgs = np.stack([synth.image("natural", 0x5EED2800 + b, W, H) for b in range(B)])
    fold = gpu_run(app, r, imgs, "row", rate, recon, batch=B)
    plain = gpu_run(app, r, imgs, "row", rate, recon, batch=B, fold=0)
    assert np.array_equal(fold, plain)
    assert np.array_equal(gpu_run(app, r, imgs, "row", rate, recon, batch=B, tile_h=37), plain)
    want = oracle.run(oracle.params(app, W, H, r, "row", rate, recon), imgs[1])
    assert_close(app, r, fold[1], want)
