"""Pins of the CPU oracle against what the paper and mathematics fix
(DESIGN.md "Pins" P1..P12).  No GPU; every check here is independent of the
oracle's own code path (closed forms, brute force, invariants, the paper's
printed computation and its reported orderings)."""
import itertools
import os

import numpy as np
import pytest

import oracle
import synth

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")

SCHEMES = ["row", "col", "checker"]
RATES = [(1, 2), (1, 3), (1, 4), (2, 3), (3, 4), (7, 8), (1, 8)]
RECONS = ["nn", "li"]


def P(app="gaussian", W=16, H=16, r=2, scheme="none", rate=(0, 1), recon="nn", G=2):
    return oracle.params(app, W, H, r, scheme, rate, recon, G)


# --------------------------------------------------------------------------
# P0: the paper's only printed computation: x1 = (x0+x2)/2
def test_p0_golden_li_midpoint():
    rows = [l.split() for l in open(os.path.join(GOLDEN, "li_midpoint_1d.txt")) if l.strip() and l[0] != "#"]
    for x0, x2, x1 in rows:
        img = np.array([[float(x0)], [123.0], [float(x2)]], dtype=np.float32)  # 1 column, rows 0..2
        p = P("gaussian", 1, 3, 1, "row", (1, 2), "li")
        R = oracle.reconstruct(p, img)
        assert R[0, 0] == float(x0) and R[2, 0] == float(x2)
        assert R[1, 0] == float(x1)
        # the same along x (column scheme, G = 1)
        p = P("gaussian", 3, 1, 1, "col", (1, 2), "li", G=1)
        R = oracle.reconstruct(p, img.reshape(1, 3).copy())
        assert R[0, 1] == float(x1)


# --------------------------------------------------------------------------
# P1: rate 0 (or scheme none) is the exact kernel, bit for bit (north_star)
@pytest.mark.parametrize("app,r", [("gaussian", 1), ("gaussian", 2), ("sobel", 1), ("sobel", 2),
                                   ("gauss_sobel", 2), ("inversion", 0)])
def test_p1_rate0_is_exact(app, r):
    img = synth.image("natural", 7, 37, 29)
    ex = oracle.run(P(app, 37, 29, r), img)
    for s in SCHEMES:
        out = oracle.run(P(app, 37, 29, r, s, (0, 4), "li"), img)
        assert np.array_equal(out, ex)


def test_p1_rate0_is_exact_median():
    img = synth.image("natural", 7, 37, 29, np.uint8)
    ex = oracle.run(P("median", 37, 29, 1), img)
    for s in SCHEMES:
        assert np.array_equal(oracle.run(P("median", 37, 29, 1, s, (0, 2), "li"), img), ex)


# --------------------------------------------------------------------------
# P2: a constant image rebuilds exactly; Gaussian = c, Sobel = 0, Median = c
@pytest.mark.parametrize("scheme,rate,recon", list(itertools.product(SCHEMES, RATES, RECONS)))
def test_p2_constant_image(scheme, rate, recon):
    W, H, c = 19, 17, 137.0
    img = np.full((H, W), c, dtype=np.float32)
    R = oracle.reconstruct(P("gaussian", W, H, 2, scheme, rate, recon, 3), img)
    assert np.all(R == c)
    for app, r, want in [("gaussian", 1, c), ("gaussian", 2, c), ("sobel", 1, 0.0), ("sobel", 2, 0.0),
                         ("gauss_sobel", 2, 0.0), ("inversion", 0, 255 - c)]:
        out = oracle.run(P(app, W, H, r, scheme, rate, recon, 3), img)
        assert np.all(out == want), app
    u = np.full((H, W), 77, dtype=np.uint8)
    assert np.all(oracle.run(P("median", W, H, 1, scheme, rate, recon, 3), u) == 77)


# --------------------------------------------------------------------------
# P3: affine ramps rebuild exactly under LI wherever both sides are loaded;
# NN is exact iff the ramp is constant along the rebuild axis.
@pytest.mark.parametrize("scheme,rate", list(itertools.product(SCHEMES, RATES)))
def test_p3_ramp_li_exact(scheme, rate):
    W, H, G = 41, 37, 3
    yy, xx = np.mgrid[0:H, 0:W]
    f = (5 + 3 * xx + 2 * yy).astype(np.float32)
    p = P("gaussian", W, H, 2, scheme, rate, "li", G)
    R = oracle.reconstruct(p, f)
    m = oracle.mask(p)
    num, den = rate
    # pixels with a loaded sample on both sides along the axis
    both = np.zeros_like(m, dtype=bool)
    for y in range(H):
        for x in range(W):
            if scheme == "col":
                line = m[y, :]
                both[y, x] = line[:x].any() and line[x + 1:].any()
            else:
                line = m[:, x]
                both[y, x] = line[:y].any() and line[y + 1:].any()
    sel = (m == 0) & both
    assert sel.sum() > 0
    assert np.array_equal(R[sel], f[sel].astype(np.float64))
    # u8 with integer round-half-up: exact too
    fu = (8 + xx + yy).astype(np.uint8)
    Ru = oracle.reconstruct(p, fu)
    assert np.array_equal(Ru[sel], fu[sel])
    # NN: exact when the ramp is constant along the axis, wrong otherwise
    pn = P("gaussian", W, H, 2, scheme, rate, "nn", G)
    g = (5 + 3 * yy).astype(np.float32) if scheme == "col" else (5 + 3 * xx).astype(np.float32)
    assert np.array_equal(oracle.reconstruct(pn, g), g.astype(np.float64))
    assert not np.array_equal(oracle.reconstruct(pn, f)[m == 0], f[m == 0])


# --------------------------------------------------------------------------
# P4: stencil weights/orientation on ramps (interior, >= r from borders)
def test_p4_stencils_on_ramps():
    W, H = 24, 20
    yy, xx = np.mgrid[0:H, 0:W]
    for beta, gamma in [(3, 0), (0, 2), (3, 4), (-5, 1)]:
        f = (600 + beta * xx + gamma * yy).astype(np.float32)
        for r, k in [(1, 8.0), (2, 128.0)]:
            g = oracle.run(P("gaussian", W, H, r), f)
            s = oracle.run(P("sobel", W, H, r), f)
            inner = (slice(r, H - r), slice(r, W - r))
            assert np.array_equal(g[inner], f[inner].astype(np.float64))
            assert np.allclose(s[inner], k * np.hypot(beta, gamma), rtol=1e-14, atol=0)
    # Sobel sign/orientation: Gx responds to x ramps only (a y ramp on a
    # 1-column image gives Gx = 0 exactly, and vice versa).
    col = (np.arange(H, dtype=np.float32) * 3).reshape(H, 1).copy()
    s = oracle.run(P("sobel", 1, H, 1), col)
    assert np.allclose(s[1:-1, 0], 8 * 3)
    # an impulse gives the binomial weights (Gaussian), up to normalisation
    imp = np.zeros((9, 9), dtype=np.float32)
    imp[4, 4] = 256.0
    g = oracle.run(P("gaussian", 9, 9, 2), imp)
    b = np.array([1, 4, 6, 4, 1], dtype=np.float64)
    assert np.array_equal(g[2:7, 2:7], np.outer(b, b))
    g1 = oracle.run(P("gaussian", 9, 9, 1), imp)
    b1 = np.array([1, 2, 1], dtype=np.float64)
    assert np.array_equal(g1[3:6, 3:6], np.outer(b1, b1) * 16)
    # Inversion: digital negative
    assert np.array_equal(oracle.run(P("inversion", 9, 9, 0), imp), 255.0 - imp.astype(np.float64))


def _np_sobel(img, r):
    """independent numpy formulation: separable correlation with edge padding"""
    s = np.array([1, 2, 1.0]) if r == 1 else np.array([1, 4, 6, 4, 1.0])
    d = np.array([-1, 0, 1.0]) if r == 1 else np.array([-1, -2, 0, 2, 1.0])
    pad = np.pad(img.astype(np.float64), r, mode="edge")
    H, W = img.shape

    def corr(a, ky, kx):
        out = np.zeros((H, W))
        for i in range(2 * r + 1):
            for j in range(2 * r + 1):
                out += ky[i] * kx[j] * a[i:i + H, j:j + W]
        return out
    gx = corr(pad, s, d)
    gy = corr(pad, d, s)
    return np.sqrt(gx * gx + gy * gy), corr(pad, s, s) / s.sum() ** 2


@pytest.mark.parametrize("r", [1, 2])
def test_p4_stencils_vs_numpy(r):
    img = synth.image("natural", 11, 33, 27)
    sob, gau = _np_sobel(img, r)
    assert np.allclose(oracle.run(P("sobel", 33, 27, r), img), sob, rtol=1e-13, atol=1e-9)
    assert np.allclose(oracle.run(P("gaussian", 33, 27, r), img), gau, rtol=1e-13, atol=1e-9)
    # fused pipeline = Sobel3(Gaussian5(.)) composed from the numpy pieces
    _, g5 = _np_sobel(img, 2)
    s3, _ = _np_sobel(g5, 1)
    assert np.allclose(oracle.run(P("gauss_sobel", 33, 27, 2), img), s3, rtol=1e-12, atol=1e-9)


# --------------------------------------------------------------------------
# P5: the median against brute force (numpy sort of the 9 clamped neighbours)
def _np_median(img):
    H, W = img.shape
    pad = np.pad(img, 1, mode="edge")
    stack = np.stack([pad[i:i + H, j:j + W] for i in range(3) for j in range(3)])
    return np.sort(stack, axis=0)[4]


def test_p5_median_brute_force():
    rng = np.random.default_rng(5)
    for _ in range(300):
        W, H = rng.integers(1, 8, size=2)
        img = rng.integers(0, 3, size=(H, W)).astype(np.uint8)
        assert np.array_equal(oracle.run(P("median", W, H, 1), img), _np_median(img))
    img = rng.integers(0, 256, size=(61, 67)).astype(np.uint8)
    assert np.array_equal(oracle.run(P("median", 67, 61, 1), img), _np_median(img))
    # perforated median = brute-force median of the rebuilt image
    for s, rate, rc in [("col", (1, 2), "nn"), ("row", (3, 4), "li"), ("checker", (1, 4), "li")]:
        p = P("median", 67, 61, 1, s, rate, rc, 4)
        assert np.array_equal(oracle.run(p, img), _np_median(oracle.reconstruct(p, img)))


# --------------------------------------------------------------------------
# P6: Hotspot -- fixed point, closed-form decay, Rodinia coefficients (closed
# forms of Rodinia's formulas at the 1024 cell size), Laplacian and clamp
def test_p6_hotspot_coefficients_closed_form():
    sdc, rx1, ry1, rz1, amb = oracle.hotspot_coeffs()
    gw = 0.016 / 1024
    # step/Cap = precision / (max_pd * gw * gh); 1/Rx = 2 k t; 1/Rz = k gw gh / t
    assert sdc == pytest.approx(0.001 / (3.0e6 * gw * gw), rel=1e-14)
    assert sdc == pytest.approx(1048.576 / 768.0, rel=1e-14)
    assert rx1 == pytest.approx(2 * 100 * 0.0005, rel=1e-14) and ry1 == pytest.approx(rx1, rel=1e-14)
    assert rz1 == pytest.approx(100 * gw * gw / 0.0005, rel=1e-14)
    assert amb == 80.0
    # the explicit scheme is stable: 1 - 2 c_x - 2 c_y - c_z > 0
    assert 1 - 4 * sdc * rx1 - sdc * rz1 > 0


def test_p6_hotspot_fixed_point_and_decay():
    sdc, rx1, ry1, rz1, amb = oracle.hotspot_coeffs()
    W, H = 13, 11
    T = np.full((H, W), 80.0, dtype=np.float32)
    Pz = np.zeros((H, W), dtype=np.float32)
    for s in ["none", "row", "col", "checker"]:
        p = P("hotspot", W, H, 1, s, (1, 2) if s != "none" else (0, 1), "li")
        assert np.array_equal(oracle.hotspot(p, T, Pz, 7), np.full((H, W), 80.0))
    T0, P0 = 330.0, 0.005
    Tu = np.full((H, W), T0, dtype=np.float32)
    Pu = np.full((H, W), P0, dtype=np.float32)
    Tstar = amb + np.float64(np.float32(P0)) / rz1
    for k in [1, 5, 40]:
        want = Tstar + (T0 - Tstar) * (1 - sdc * rz1) ** k
        out = oracle.hotspot(P("hotspot", W, H, 1, "row", (3, 4), "nn"), Tu, Pu, k)
        assert np.allclose(out, want, rtol=1e-12, atol=0)


def test_p6_hotspot_laplacian_and_clamp():
    sdc, rx1, ry1, rz1, amb = oracle.hotspot_coeffs()
    W, H = 12, 10
    yy, xx = np.mgrid[0:H, 0:W]
    a, b = 0.25, 0.5
    T = (300 + a * xx * xx + b * yy * yy).astype(np.float32)  # exact in fp32
    Pz = np.full((H, W), 0.0078125, dtype=np.float32)
    out = oracle.hotspot(P("hotspot", W, H, 1), T, Pz, 1)
    T64 = T.astype(np.float64)
    inner = (slice(1, H - 1), slice(1, W - 1))
    want = T64 + sdc * (0.0078125 + 2 * b * ry1 + 2 * a * rx1 + (amb - T64) * rz1)
    assert np.allclose(out[inner], want[inner], rtol=1e-14, atol=0)
    # clamp: on a linear x ramp the Laplacian vanishes inside and equals the
    # one-sided difference at x = 0 and x = W-1
    L = (300 + 2 * xx).astype(np.float32)
    out = oracle.hotspot(P("hotspot", W, H, 1), L, Pz, 1).astype(np.float64)
    L64 = L.astype(np.float64)
    base = L64 + sdc * (0.0078125 + (amb - L64) * rz1)
    assert np.allclose(out[:, 1:-1], base[:, 1:-1], rtol=1e-14)
    assert np.allclose(out[:, 0], base[:, 0] + sdc * 2 * rx1, rtol=1e-14)
    assert np.allclose(out[:, -1], base[:, -1] - sdc * 2 * rx1, rtol=1e-14)


# --------------------------------------------------------------------------
# P7: the error metric
def test_p7_error_metric():
    rng = np.random.default_rng(7)
    e = rng.integers(1, 200, size=1000).astype(np.float64)
    assert oracle.error("mre", e, e) == (0.0, 1000)
    assert oracle.error("mre", e, e * (1 + 2.0 ** -4))[0] == 2.0 ** -4
    assert oracle.error("mre", e, e * (1 - 2.0 ** -3))[0] == 2.0 ** -3
    assert oracle.error("mre", e, np.zeros_like(e))[0] == 1.0
    e0 = e.copy()
    e0[::4] = 0  # zero true values are excluded from the MRE
    v, c = oracle.error("mre", e0, e0 + 1.0)
    assert c == 750 and v == pytest.approx(np.mean(1.0 / e0[e0 != 0]), rel=1e-14)
    v, c = oracle.error("me", e, e + 2.0)
    assert v == pytest.approx(2000.0 / e.sum(), rel=1e-14)
    v, c = oracle.error("mae", e, e - 3.0)
    assert v == 3.0 and c == 1000
    u = e.astype(np.uint8)
    assert oracle.error("mre", u, u)[0] == 0.0
    f = e.astype(np.float32)
    assert oracle.error("mre", f, f * np.float32(1.0625))[0] == 2.0 ** -4


# --------------------------------------------------------------------------
# P8: an independent brute-force formulation of mask + rebuild (explicit
# enumeration of the loaded set, argmin distance, lower-coordinate tie)
def _bf_mask(scheme, num, den, G, W, H):
    if scheme == "none" or num == 0:
        return np.ones((H, W), dtype=bool)
    if num == den - 1:
        kept_phases = {0}
    else:
        kept_phases = set(range(den)) - {den - 1}
    m = np.zeros((H, W), dtype=bool)
    for y in range(H):
        for x in range(W):
            cell = {"row": y, "col": x // G, "checker": x // G + y}[scheme]
            m[y, x] = (cell % den) in kept_phases
    return m


def _bf_rebuild(scheme, recon, m, img):
    H, W = img.shape
    out = img.astype(np.float64).copy() if img.dtype != np.uint8 else img.astype(np.int64).copy()
    for y in range(H):
        for x in range(W):
            if m[y, x]:
                continue
            if scheme == "col":
                cands = [(abs(x - xx), xx < x, img[y, xx]) for xx in range(W) if m[y, xx]]
            else:
                cands = [(abs(y - yy), yy < y, img[yy, x]) for yy in range(H) if m[yy, x]]
            below = [c for c in cands if c[1]]
            above = [c for c in cands if not c[1]]
            a = min(below, key=lambda c: c[0]) if below else None
            b = min(above, key=lambda c: c[0]) if above else None
            if recon == "li" and a and b:
                da, db = a[0], b[0]
                if img.dtype == np.uint8:
                    out[y, x] = (int(a[2]) * db + int(b[2]) * da + (da + db) // 2) // (da + db)
                else:
                    out[y, x] = (float(a[2]) * db + float(b[2]) * da) / (da + db)
            else:
                best = min([c for c in (a, b) if c], key=lambda c: (c[0], not c[1]))
                out[y, x] = best[2]
    return out


def test_p8_brute_force_rebuild():
    rng = np.random.default_rng(8)
    n = 0
    for W in range(1, 10):
        for H in range(1, 10):
            for scheme in SCHEMES:
                for num, den in [(1, 2), (1, 3), (2, 3), (1, 4), (3, 4), (7, 8)]:
                    if scheme == "checker" and H < den:
                        continue  # rejected configuration (no loaded sample on some column)
                    G = int(rng.integers(1, 4))
                    for recon in RECONS:
                        if rng.random() > 0.35:
                            continue
                        p = P("gaussian", W, H, 1, scheme, (num, den), recon, G)
                        m = _bf_mask(scheme, num, den, G, W, H)
                        assert np.array_equal(oracle.mask(p).astype(bool), m)
                        f = rng.integers(8, 248, size=(H, W)).astype(np.float32)
                        assert np.array_equal(oracle.reconstruct(p, f), _bf_rebuild(scheme, recon, m, f))
                        u = f.astype(np.uint8)
                        assert np.array_equal(oracle.reconstruct(p, u).astype(np.int64),
                                              _bf_rebuild(scheme, recon, m, u))
                        n += 1
    assert n > 300


# --------------------------------------------------------------------------
# P9: windowed / per-pixel formulations equal the whole-image definition
# (the dependency-cone reading that band sharding relies on)
@pytest.mark.parametrize("scheme,rate,recon", [("none", (0, 1), "nn"), ("row", (1, 2), "li"),
                                               ("row", (3, 4), "nn"), ("col", (1, 4), "li"),
                                               ("checker", (1, 2), "li")])
def test_p9_hotspot_rect_equals_full(scheme, rate, recon):
    W, H = 40, 36
    T, Pw = synth.hotspot(synth.SEED_C4, W, H)
    p = P("hotspot", W, H, 1, scheme, rate, recon, 2)
    full = oracle.hotspot(p, T, Pw, 6)
    for x0, y0, w, h in [(0, 0, 5, 4), (17, 13, 6, 5), (35, 30, 5, 6), (10, 0, 3, 36)]:
        assert np.array_equal(oracle.hotspot_rect(p, T, Pw, 6, x0, y0, w, h), full[y0:y0 + h, x0:x0 + w])


@pytest.mark.parametrize("app,r", [("gaussian", 2), ("sobel", 1), ("gauss_sobel", 2), ("median", 1),
                                   ("inversion", 0)])
def test_p9_pixel_equals_full(app, r):
    W, H = 45, 31
    u8 = app == "median"
    img = synth.image("natural", 3, W, H, np.uint8 if u8 else np.float32)
    rng = np.random.default_rng(9)
    for scheme, rate, recon in [("row", (1, 2), "li"), ("col", (3, 4), "nn"), ("checker", (1, 4), "li")]:
        p = P(app, W, H, r, scheme, rate, recon, 4)
        full = oracle.run(p, img)
        xs = np.r_[0, W - 1, rng.integers(0, W, 30)]
        ys = np.r_[0, H - 1, rng.integers(0, H, 30)]
        assert np.array_equal(oracle.run_pixels(p, img, xs, ys), full[ys, xs])


# --------------------------------------------------------------------------
# P10: homogeneity -- scaling the input by 2^k scales Gaussian, Median and LI
# outputs exactly and leaves the MRE unchanged
def test_p10_scaling():
    img = synth.image("natural", 4, 30, 26)
    for scheme, rate in [("row", (1, 2)), ("col", (1, 3)), ("checker", (3, 4))]:
        p = P("gaussian", 30, 26, 2, scheme, rate, "li", 2)
        ex = oracle.run(P("gaussian", 30, 26, 2), img)
        a = oracle.run(p, img)
        a4 = oracle.run(p, img * 4)
        assert np.array_equal(a4, a * 4)
        assert oracle.error("mre", ex, a)[0] == oracle.error("mre", ex * 4, a4)[0]
    u = (synth.image("natural", 4, 30, 26, np.uint8) // 2).astype(np.uint8)
    p = P("median", 30, 26, 1, "row", (1, 2), "nn")
    assert np.array_equal(oracle.run(p, u * 2), oracle.run(p, u) * 2)


# --------------------------------------------------------------------------
# P11: the paper's reported orderings on synthetic stand-ins (Sec. 6.3, Fig. 8,
# PAPER.md:822-834; Fig. 7)
def test_p11_paper_orderings():
    W = H = 256
    nat = synth.image("natural", synth.SEED_C2 + 1, W, H)
    for app in ["gaussian", "inversion"]:
        r = 2 if app == "gaussian" else 0
        ex = oracle.run(P(app, W, H, r), nat)

        def err(rate, rc, s="row"):
            return oracle.error("mre", ex, oracle.run(P(app, W, H, r, s, rate, rc), nat))[0]
        rows1_nn, rows2_nn, rows1_li = err((1, 2), "nn"), err((3, 4), "nn"), err((1, 2), "li")
        # "the error is higher if the approximation scheme is more aggressive" (:822-823)
        assert rows2_nn > rows1_nn
        # "The error for Rows1:LI is smaller than for Rows1:NN" (:830-832)
        assert rows1_li < rows1_nn
        # "the error of Rows1:NN is already small and less than 4%" (:832-833)
        assert rows1_nn < 0.04
    # median: flat < natural < pattern (Fig. 7: 0.12% / 5.05% / 19.32%)
    errs = []
    for cls in ["flat", "natural", "pattern"]:
        u = synth.image(cls, 99, W, H, np.uint8)
        ex = oracle.run(P("median", W, H, 1), u)
        errs.append(oracle.error("mre", ex, oracle.run(P("median", W, H, 1, "row", (1, 2), "nn"), u))[0])
    assert errs[0] < errs[1] < errs[2]


# --------------------------------------------------------------------------
# P12: the synthetic generator is deterministic and in range
def test_p12_synth_ranges():
    for cls in ["flat", "natural", "pattern"]:
        a = synth.image(cls, 123, 200, 150)
        b = synth.image(cls, 123, 200, 150)
        assert np.array_equal(a, b)
        assert a.min() >= 8 and a.max() <= 247 and np.all(a == np.round(a))
        assert np.array_equal(synth.image(cls, 123, 200, 150, np.uint8), a.astype(np.uint8))
    T, Pw = synth.hotspot(5, 64, 48)
    assert np.all(T * 64 == np.round(T * 64)) and T.min() > 300 and T.max() < 340
    assert Pw.min() >= 0 and np.all(Pw * 131072 == np.round(Pw * 131072))


# --------------------------------------------------------------------------
# P13: Stencil1 (PAPER.md:479-490, Fig. 5; :819-821) -- the tile fetches only
# its interior, the halo is rebuilt by NN from the tile border
def _np_stencil1(app, r, img, tw, th):
    """independent formulation: pad every tile with its own border, filter it"""
    H, W = img.shape
    out = np.zeros((H, W))
    for ty in range(0, H, th):
        for tx in range(0, W, tw):
            t = img[ty:ty + th, tx:tx + tw]
            if app == "median":
                out[ty:ty + th, tx:tx + tw] = _np_median(t)
            else:
                sob, gau = _np_sobel(t, r)
                out[ty:ty + th, tx:tx + tw] = sob if app == "sobel" else gau
    return out


@pytest.mark.parametrize("app,r", [("gaussian", 1), ("gaussian", 2), ("sobel", 1), ("sobel", 2), ("median", 1)])
@pytest.mark.parametrize("tile", [(16, 16), (32, 8), (8, 4), (5, 7)])
def test_p13_stencil1_per_tile(app, r, tile):
    W, H = 53, 41
    img = synth.image("natural", 13, W, H, np.uint8 if app == "median" else np.float32)
    p = P(app, W, H, r, "stencil1", (0, 1), "nn")
    p.tile_w, p.tile_h = tile
    got = oracle.run(p, img)
    want = _np_stencil1(app, r, img, *tile)
    if app == "median":
        assert np.array_equal(got, want)
    else:
        assert np.allclose(got, want, rtol=1e-13, atol=1e-9)
    xs, ys = np.arange(0, W, 3), np.arange(0, H, 3)[: len(np.arange(0, W, 3))]
    xs = xs[: len(ys)]
    assert np.array_equal(oracle.run_pixels(p, img, xs, ys), got[ys, xs])


def test_p13_stencil1_invariants():
    W, H = 40, 30
    img = synth.image("natural", 14, W, H)
    p = P("gaussian", W, H, 2, "stencil1")
    p.tile_w, p.tile_h = 64, 64  # one tile covers the image: exact
    assert np.array_equal(oracle.run(p, img), oracle.run(P("gaussian", W, H, 2), img))
    c = np.full((H, W), 61.0, dtype=np.float32)
    p.tile_w, p.tile_h = 8, 8
    assert np.all(oracle.run(p, c) == 61.0)
    ps = P("sobel", W, H, 1, "stencil1")
    ps.tile_w, ps.tile_h = 8, 8
    assert np.all(oracle.run(ps, c) == 0.0)
    # interior pixels of a tile (>= r from its border) are exact
    ex = oracle.run(P("gaussian", W, H, 2), img)
    st = oracle.run(p, img)
    inner = np.zeros((H, W), bool)
    for ty in range(0, H, 8):
        for tx in range(0, W, 8):
            inner[ty + 2:min(ty + 6, H - 2), tx + 2:min(tx + 6, W - 2)] = True
    assert np.array_equal(st[inner], ex[inner]) and not np.array_equal(st, ex)


def test_p13_stencil1_paper_claims():
    """'The error for Stencil1 is very low and always less than 1%' and below
    Rows1:NN, on a natural-image stand-in"""
    W = H = 256
    img = synth.image("natural", synth.SEED_C2 + 1, W, H)
    ex = oracle.run(P("gaussian", W, H, 1), img)
    p = P("gaussian", W, H, 1, "stencil1")
    p.tile_w, p.tile_h = 16, 16
    e_s1 = oracle.error("mre", ex, oracle.run(p, img))[0]
    e_r1 = oracle.error("mre", ex, oracle.run(P("gaussian", W, H, 1, "row", (1, 2), "nn"), img))[0]
    assert e_s1 < 0.01 and e_s1 < e_r1


# --------------------------------------------------------------------------
# P14: Hotspot temporal blocking (R19): with tblock
# = p, T is perforated and rebuilt only at steps it % p == 0 -- the steps a
# p-step-per-launch kernel loads T from memory; the others read on-chip T.
def _np_hotspot(T0, P0, iters, den, num, recon, tblock):
    """independent numpy formulation: explicit kept-row list, np.pad(edge)
    clamp, Rodinia update in fp64"""
    sdc, rx1, ry1, rz1, amb = oracle.hotspot_coeffs()
    H, W = T0.shape
    keep_one = num == den - 1
    kept = [y for y in range(H) if (y % den == 0 if keep_one else y % den != den - 1)]

    def rebuild(A):
        R = A.copy()
        for y in range(H):
            if y in kept:
                continue
            lo = [k for k in kept if k < y]
            hi = [k for k in kept if k > y]
            a, b = (lo[-1] if lo else None), (hi[0] if hi else None)
            if recon == "li" and a is not None and b is not None:
                R[y] = (A[a] * (b - y) + A[b] * (y - a)) / (b - a)
            elif b is None or (a is not None and y - a <= b - y):
                R[y] = A[a]
            else:
                R[y] = A[b]
        return R

    T = T0.astype(np.float64)
    Pr = rebuild(P0.astype(np.float64))
    for it in range(iters):
        Tr = rebuild(T) if it % tblock == 0 else T
        Q = np.pad(Tr, 1, mode="edge")
        lap_y = Q[2:, 1:-1] + Q[:-2, 1:-1] - 2 * Tr
        lap_x = Q[1:-1, 2:] + Q[1:-1, :-2] - 2 * Tr
        T = Tr + sdc * (Pr + lap_y * ry1 + lap_x * rx1 + (amb - Tr) * rz1)
    return T


@pytest.mark.parametrize("rate,recon", [((1, 2), "li"), ((1, 2), "nn"), ((3, 4), "li"), ((1, 3), "nn")])
@pytest.mark.parametrize("tblock", [1, 2, 3, 8])
def test_p14_hotspot_tblock_vs_numpy(rate, recon, tblock):
    W, H, iters = 9, 13, 7
    T, Pw = synth.hotspot(11, W, H)
    p = oracle.params("hotspot", W, H, 1, "row", rate, recon, 8, tblock=tblock)
    got = oracle.hotspot(p, T, Pw, iters)
    want = _np_hotspot(T, Pw, iters, rate[1], rate[0], recon, tblock)
    assert np.allclose(got, want, rtol=1e-13, atol=0)


def test_p14_hotspot_tblock_invariants():
    sdc, rx1, ry1, rz1, amb = oracle.hotspot_coeffs()
    W, H = 12, 10
    T, Pw = synth.hotspot(5, W, H)
    base = oracle.hotspot(oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8), T, Pw, 6)
    # tblock 1 (and 0) is the per-step definition
    for tb in (0, 1):
        p = oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8, tblock=tb)
        assert np.array_equal(oracle.hotspot(p, T, Pw, 6), base)
    # rate 0 is exact whatever tblock
    ex = oracle.hotspot(oracle.params("hotspot", W, H, 1), T, Pw, 6)
    assert np.array_equal(oracle.hotspot(oracle.params("hotspot", W, H, 1, tblock=3), T, Pw, 6), ex)
    # fixed point and the uniform closed-form decay hold for any tblock
    T0, P0 = 330.0, 0.005
    Tu = np.full((H, W), T0, dtype=np.float32)
    Pu = np.full((H, W), P0, dtype=np.float32)
    Tstar = amb + np.float64(np.float32(P0)) / rz1
    for tb in (2, 5):
        p = oracle.params("hotspot", W, H, 1, "row", (3, 4), "li", 8, tblock=tb)
        assert np.array_equal(oracle.hotspot(p, np.full((H, W), 80.0, np.float32), np.zeros((H, W), np.float32), 7),
                              np.full((H, W), 80.0))
        assert np.allclose(oracle.hotspot(p, Tu, Pu, 9), Tstar + (T0 - Tstar) * (1 - sdc * rz1) ** 9, rtol=1e-12)
    # tblock >= iters perforates T once: equals 1 perforated step then exact steps
    p1 = oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8)
    T64 = T.astype(np.float64)
    oracle.hotspot_window(p1, T64, Pw, 0, 0, 1)
    oracle.hotspot_window(oracle.params("hotspot", W, H, 1, "none", (0, 1), "nn", 8), T64,
                          oracle.reconstruct(p1, Pw).astype(np.float32), 0, 0, 5)
    got = oracle.hotspot(oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8, tblock=6), T, Pw, 6)
    assert np.allclose(got, T64, rtol=1e-13)


def test_p14_hotspot_tblock_perforates_less():
    """fewer perforated loads -> error against the exact run does not grow
    (synthetic C4-like grid, 24 steps)"""
    W, H = 96, 64
    T, Pw = synth.hotspot(synth.SEED_C4, W, H)
    ex = oracle.hotspot(oracle.params("hotspot", W, H, 1), T, Pw, 24)
    errs = [oracle.error("mre", ex, oracle.hotspot(oracle.params("hotspot", W, H, 1, "row", (1, 2), "li", 8,
                                                                 tblock=tb), T, Pw, 24))[0] for tb in (1, 4, 24)]
    assert errs[0] > errs[1] > errs[2] > 0
