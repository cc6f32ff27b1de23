"""GPU <-> oracle parity in the EXACT launch configurations bench.py times.

bench.py's C2 step is one perf_run over 8 frames of 4096^2 fp32 with 128-B
cells; that batch is large enough for the launcher's fixed 16- / 24-row
segments (kernel.cuh launch_one), which the small parity shapes never reach.  These
tests build the bench's plans (same CONFIGS, batch, granule, seeds, device
generator), run them once, and compare against oracle.run_pixels:

* whole rows at and around segment boundaries the launcher can pick
  (y = 0..2, 14..18, 22..26, 46..50, 62..66, 126..130 and the last rows) on
  one frame;
* whole columns at and around the 1024-column strip boundaries (x = 1022..1026)
  and the image's right edge on another frame -- every row, so every segment
  boundary of any segment height is crossed;
* the four image corners of every sampled frame.

Tolerance: north_star's 1e-5 relative per element (Sobel's cancellation floor
as in test_gpu_parity.py); the u8 median bit-exact.  C2 covers all 36 timed
variants (Gaussian5 / Sobel3 x row/col/checker x NN/LI x 1/2, 1/4, 3/4).
"""
import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_cgo_maiercj18_b200 as kp  # noqa: E402
from bench import CONFIGS  # noqa: E402  (the bench's own workload table)

from test_gpu_parity import assert_close  # noqa: E402

G_BYTES = 128  # bench.py: the measured DRAM fill granule


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    torch.cuda.init()


def _frames(cfg, B):
    u8 = cfg["app"] == "median"
    x = torch.empty((B, cfg["H"], cfg["W"]), dtype=torch.uint8 if u8 else torch.float32, device="cuda")
    synth.image_device(cfg["cls"], cfg["seed"], cfg["W"], cfg["H"], B, x.data_ptr(), u8)
    return x


def _boundary_rows(H):
    ys = {0, 1, 2, H - 3, H - 2, H - 1}
    for b in (16, 24, 48, 64, 128):  # fixed 16 / 24-row segments, wave-filling heights
        ys |= {b - 2, b - 1, b, b + 1, b + 2}
    ys |= {H // 2 - 1, H // 2}
    return sorted(y for y in ys if 0 <= y < H)


def _boundary_cols(W, tw):
    xs = {0, 1, W - 2, W - 1}
    for b in range(tw, W, tw):
        xs |= {b - 2, b - 1, b, b + 1, b + 2}
    return sorted(x for x in xs if 0 <= x < W)


def _check_frame(app, r, prm, img, got, W, H, tw, rows=True, cols=True, xstep=1, max_strip_cols=None):
    if rows:  # (xstep coprime to the 16-column lane chunk still visits every lane position)
        ys = _boundary_rows(H)
        yy, xx = np.meshgrid(ys, np.arange(0, W, xstep), indexing="ij")
        want = oracle.run_pixels(prm, img, xx.ravel(), yy.ravel())
        assert_close(app, r, got[yy.ravel(), xx.ravel()], want)
    if cols:
        xs = _boundary_cols(W, tw)
        if max_strip_cols:  # (the u8 frames are 8192 rows tall: the first strip boundary + the image edges)
            xs = [x for x in xs if x < 2 or x >= W - 2 or abs(x - tw) <= 2][:max_strip_cols]
        xx, yy = np.meshgrid(xs, np.arange(H), indexing="ij")
        want = oracle.run_pixels(prm, img, xx.ravel(), yy.ravel())
        assert_close(app, r, got[yy.ravel(), xx.ravel()], want)


C2_VARIANTS = [(app, r, s, rate, rc) for app, r in (("gaussian", 2), ("sobel", 1))
               for s in ("row", "col", "checker") for rate in ((1, 2), (1, 4), (3, 4)) for rc in ("nn", "li")]


@pytest.fixture(scope="module")
def c2_frames():
    cfg = CONFIGS["C2"]
    x = _frames(cfg, cfg["batch"])
    torch.cuda.synchronize()
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    imgs = {f: synth.image(cfg["cls"], cfg["seed"] + f, W, H) for f in (0, B - 1)}
    return cfg, x, imgs


@pytest.mark.parametrize("app,r,scheme,rate,recon", C2_VARIANTS)
def test_c2_bench_launch(c2_frames, app, r, scheme, rate, recon):
    cfg, x, imgs = c2_frames
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    y = torch.empty_like(x)
    with kp.Plan(app, W, H, r, scheme, rate, recon, batch=B, granule_bytes=G_BYTES) as p:
        p.run(x, y)
    torch.cuda.synchronize()
    prm = oracle.params(app, W, H, r, scheme, rate, recon, G_BYTES // 4)
    _check_frame(app, r, prm, imgs[0], y[0].cpu().numpy(), W, H, 1024, rows=True, cols=False)
    _check_frame(app, r, prm, imgs[B - 1], y[B - 1].cpu().numpy(), W, H, 1024, rows=False, cols=True)


def test_c2_bench_exact_and_error(c2_frames):
    """the bench's exact kernel (speedup denominator) and its error figure on the
    same batch: exact == oracle at the boundaries; perf_error(batch) == the
    oracle's metric on the same two buffers (frame 0 checked whole)"""
    cfg, x, imgs = c2_frames
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    yex = torch.empty_like(x)
    y = torch.empty_like(x)
    with kp.Plan("gaussian", W, H, 2, "none", (0, 1), "nn", batch=B) as pe, \
            kp.Plan("gaussian", W, H, 2, "row", (1, 2), "li", batch=B, granule_bytes=G_BYTES) as p:
        pe.run(x, yex)
        p.run(x, y)
        v, c = p.error(yex, y)
    torch.cuda.synchronize()
    prm = oracle.params("gaussian", W, H, 2, "none", (0, 1), "nn")
    _check_frame("gaussian", 2, prm, imgs[0], yex[0].cpu().numpy(), W, H, 1024, cols=False)
    ov, oc = oracle.error("mre", yex.cpu().numpy().reshape(-1), y.cpu().numpy().reshape(-1))
    assert c == oc and abs(v - ov) <= 1e-9 * max(1.0, ov)


@pytest.mark.parametrize("rate", [(1, 2), (1, 4), (3, 4)])
def test_c3_bench_launch(rate):
    cfg = CONFIGS["C3"]
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    x = _frames(cfg, B)
    y = torch.empty_like(x)
    with kp.Plan("median", W, H, 1, "col", rate, "nn", batch=B, granule_bytes=G_BYTES) as p:
        p.run(x, y)
    torch.cuda.synchronize()
    prm = oracle.params("median", W, H, 1, "col", rate, "nn", G_BYTES)
    for f, rows, cols in ((0, True, False), (B - 1, False, True)):
        img = synth.image(cfg["cls"], cfg["seed"] + f, W, H, np.uint8)
        _check_frame("median", 1, prm, img, y[f].cpu().numpy(), W, H, 2048, rows=rows, cols=cols, xstep=3,
                     max_strip_cols=9)


@pytest.mark.parametrize("scheme,rate,recon", [("row", (1, 2), "li"), ("row", (3, 4), "nn"), ("none", (0, 1), "nn")])
def test_c5_bench_launch(scheme, rate, recon):
    cfg = CONFIGS["C5"]
    W, H, B = cfg["W"], cfg["H"], cfg["batch"]
    x = _frames(cfg, B)
    y = torch.empty_like(x)
    with kp.Plan("gauss_sobel", W, H, 2, scheme, rate, recon, batch=B) as p:
        p.run(x, y)
    torch.cuda.synchronize()
    prm = oracle.params("gauss_sobel", W, H, 2, scheme, rate, recon)
    for f, rows, cols in ((0, True, False), (B - 1, False, True)):
        img = synth.image(cfg["cls"], cfg["seed"] + f, W, H)
        _check_frame("gauss_sobel", 2, prm, img, y[f].cpu().numpy(), W, H, 1024, rows=rows, cols=cols)


def test_c4_bench_launch_cones():
    """C4 as bench.py runs it on one GPU: 16384^2, 200 steps, row 1/2 LI;
    the oracle on the dependency cones of patches at the corners, edges and
    strip / segment boundaries"""
    cfg = CONFIGS["C4"]
    W = H = cfg["W"]
    iters = cfg["iters"]
    T = torch.empty((H, W), device="cuda")
    P = torch.empty((H, W), device="cuda")
    synth.hotspot_band_device(cfg["seed"], W, H, 0, H, T.data_ptr(), P.data_ptr())
    out = torch.empty_like(T)
    with kp.Plan("hotspot", W, H, 1, cfg["scheme"], cfg["rate"], cfg["recon"], iters=iters) as p:
        p.hotspot(T, P, out)
    torch.cuda.synchronize()
    Th, Ph = T.cpu().numpy(), P.cpu().numpy()
    o = out.cpu().numpy()
    prm = oracle.params("hotspot", W, H, 1, cfg["scheme"], cfg["rate"], cfg["recon"])
    for x0, y0 in [(0, 0), (W - 4, H - 3), (1021, 62), (8190, 8190), (0, 127), (W - 4, 5000)]:
        want = oracle.hotspot_rect(prm, Th, Ph, iters, x0, y0, 4, 3)
        assert_close("hotspot", 1, o[y0:y0 + 3, x0:x0 + 4], want)
