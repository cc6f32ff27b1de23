"""CPU checks of the boundary: the C-ABI library loads and exports every symbol
include/kperf.h declares; plan validation (no device work) behaves as the
header documents."""
import os
import re

import pytest

import paper_conf_cgo_maiercj18_b200 as kp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def header_symbols():
    src = open(os.path.join(ROOT, "include", "kperf.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(perf_[a-z0-9_]+)\s*\(", src)))


def test_library_exports_every_header_symbol():
    L = kp.lib()
    syms = header_symbols()
    assert len(syms) >= 12
    for s in syms:
        assert hasattr(L, s), s
    assert sorted(kp.SYMBOLS) == syms


def test_version_string():
    assert "sm_100a" in kp.perf_version()


@pytest.mark.parametrize("args,status", [
    (("gaussian", 0, 10, 2, "row", (1, 2), "nn"), 1),      # W < 1
    (("gaussian", 10, 10, 3, "row", (1, 2), "nn"), 1),     # radius
    (("median", 10, 10, 2, "row", (1, 2), "nn"), 1),       # radius
    (("inversion", 10, 10, 1, "none", (0, 1), "nn"), 1),   # radius
    (("gaussian", 10, 10, 2, "row", (2, 5), "nn"), 1),     # num not in {0,1,den-1}
    (("gaussian", 10, 10, 2, "row", (1, 9), "nn"), 1),     # den > 8
    (("gaussian", 10, 10, 2, "none", (1, 2), "nn"), 1),    # none with num > 0
    (("gaussian", 10, 3, 2, "checker", (1, 4), "nn"), 1),  # checker needs H >= den
])
def test_plan_validation(args, status):
    with pytest.raises(kp.PerfError) as ei:
        kp.perf_plan(*args)
    assert ei.value.status == status


def test_plan_keys_roundtrip():
    h = kp.perf_plan("gaussian", 64, 48, 2, "col", (1, 4), "li")
    try:
        assert kp.perf_plan_get(h, "granule_bytes") == 128
        kp.perf_plan_set(h, "granule_bytes", 64)
        kp.perf_plan_set(h, "batch", 3)
        kp.perf_plan_set(h, "tile_h", 17)
        assert kp.perf_plan_get(h, "granule_bytes") == 64
        assert kp.perf_plan_get(h, "batch") == 3
        assert kp.perf_plan_get(h, "tile_h") == 17
        assert kp.perf_plan_get(h, "metric") == 0
        with pytest.raises(kp.PerfError):
            kp.perf_plan_set(h, "granule_bytes", 6)  # not a multiple of sizeof(float)
        with pytest.raises(kp.PerfError):
            kp.perf_plan_set(h, 999, 1)
    finally:
        kp.perf_destroy(h)
    hs = kp.perf_plan("sobel", 8, 8, 1, "row", (1, 2), "nn")
    assert kp.perf_plan_get(hs, "metric") == 1  # Sobel's mean error
    kp.perf_destroy(hs)


def test_product_does_not_import_oracle():
    """The product package must not reference oracle/ (independence)."""
    pkg = os.path.join(ROOT, "paper_conf_cgo_maiercj18_b200")
    for dp, _, fs in os.walk(pkg):
        for f in fs:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                txt = open(os.path.join(dp, f)).read()
                assert "import oracle" not in txt and "kperf_oracle" not in txt, f


@pytest.mark.parametrize("scheme,rate,W,gbytes,want", [
    ("checker", (3, 4), 2048, 128, 1),   # keep-one, every warp on the fast path
    ("checker", (1, 2), 2048, 32, 1),    # den 2 is keep-one too
    ("checker", (3, 4), 512, 128, 1),    # narrow image: 2 consumer warps per CTA
    ("checker", (1, 2), 2048, 4096, 0),  # 1024-px cells: the packed slot would be wider than a full one
    ("checker", (1, 4), 2048, 128, 0),   # skip-one: full-width slots
    ("checker", (3, 4), 2050, 128, 0),   # W not a multiple of the warp width
    ("row", (1, 2), 2048, 128, 0),
])
def test_checker_compact_slot_gate(scheme, rate, W, gbytes, want):
    """PERF_KEY_CHK_COMPACT (read-only) reports the layout perf_run would use;
    host-only geometry, no device work."""
    with kp.Plan("gaussian", W, 64, 2, scheme, rate, "li", granule_bytes=gbytes) as p:
        assert p.get("chk_compact") == want
        with pytest.raises(kp.PerfError):
            p.set("chk_compact", 1)


def test_binding_checks_buffers():
    """The binding refuses buffers the C ABI could not check: wrong dtype,
    non-contiguous views, wrong element counts, host arrays for device calls."""
    import numpy as np
    import torch
    with kp.Plan("gaussian", 16, 8, 2, "row", (1, 2), "li", batch=2) as p:
        with pytest.raises(TypeError):
            p.run(torch.zeros((2, 8, 16), dtype=torch.float64), torch.zeros((2, 8, 16)))
        with pytest.raises(ValueError):
            p.run(torch.zeros((2, 16, 8)).transpose(1, 2), torch.zeros((2, 8, 16)))
        with pytest.raises(ValueError):
            p.run(torch.zeros((1, 8, 16)), torch.zeros((1, 8, 16)))
        with pytest.raises(ValueError):
            p.run(np.zeros((2, 8, 16), np.float32), np.zeros((2, 8, 16), np.float32))  # device call
        with pytest.raises(ValueError):
            p.run(torch.zeros((2, 8, 16)), torch.zeros((2, 8, 16)))  # CPU tensors
    with kp.Plan("median", 16, 8, 1, "col", (1, 2), "nn") as p:
        with pytest.raises(TypeError):
            p.run_host(np.zeros((8, 16), np.float32), np.zeros((8, 16), np.uint8))


@pytest.mark.parametrize("app,r,scheme,rate,tb,want", [
    ("gaussian", 2, "row", (1, 2), 1, 4),       # radius 2 + den 2
    ("gaussian", 2, "col", (1, 2), 1, 2),       # horizontal rebuild: radius only
    ("sobel", 1, "checker", (3, 4), 1, 5),
    ("median", 1, "row", (1, 4), 1, 5),
    ("gauss_sobel", 2, "row", (3, 4), 1, 7),    # 2 + 1 + den
    ("gauss_sobel", 2, "none", (0, 1), 1, 3),
    ("hotspot", 1, "row", (1, 2), 1, 3),
    ("hotspot", 1, "row", (1, 2), 4, 6),        # TBLOCK steps per launch
])
def test_band_halo_plan(app, r, scheme, rate, tb, want):
    """perf_band_halo: host-only bookkeeping shared by the NCCL exchange, the
    single-device emulation and the gloo tests"""
    H, n = 100, 3
    cuts = kp.band_cuts(H, n)
    for rank in range(n):
        h = cuts[rank + 1] - cuts[rank]
        with kp.Plan(app, 64, h, r, scheme, rate, "li", global_h=H, band_y0=cuts[rank], tblock=tb) as p:
            hp = kp.perf_band_halo(p.handle, rank, n)
        assert hp["halo_rows"] == want and hp["buf_rows"] == h + 2 * want
        assert hp["up_rank"] == (rank - 1 if rank > 0 else -1)
        assert hp["down_rank"] == (rank + 1 if rank < n - 1 else -1)
        assert (hp["send_up_row"], hp["recv_up_row"]) == (want, 0)
        assert (hp["send_down_row"], hp["recv_down_row"]) == (h, h + want)
    with kp.Plan(app, 64, 10, r, scheme, rate, "li", global_h=H, band_y0=50) as p:
        with pytest.raises(kp.PerfError):  # an interior band cannot be rank 0
            kp.perf_band_halo(p.handle, 0, 3)


@pytest.mark.parametrize("metric,sums,want", [
    ("mre", (3.0, 99.0, 12.0), (0.25, 12)),
    ("me", (3.0, 12.0, 40.0), (0.25, 40)),
    ("mae", (10.0, 0.0, 40.0), (0.25, 40)),
    ("mre", (0.0, 0.0, 0.0), (0.0, 0)),
    ("me", (5.0, 0.0, 7.0), (0.0, 7)),
])
def test_error_finish(metric, sums, want):
    """perf_error_finish (host only): the metric from (summed) partial sums,
    PAPER.md:576-584 -- MRE and MAE divide by the count, ME by sum |e|"""
    with kp.Plan("gaussian", 8, 8, 2, metric=kp.METRIC[metric]) as p:
        assert kp.perf_error_finish(p.handle, sums) == want


@pytest.mark.parametrize("scheme,rate,H,rows", [
    ("row", (1, 2), 200, 100),   # Rows1: even rows
    ("row", (3, 4), 202, 51),    # Rows2 (keep-one): rows = 0 mod 4
    ("row", (1, 4), 202, 152),   # skip-one: rows = 3 mod 4 skipped (50 of them)
    ("row", (0, 1), 202, 202),   # rate 0: exact
    ("col", (1, 2), 202, 202),   # cells: whole rows cross PCIe
])
def test_host_h2d_bytes(scheme, rate, H, rows):
    """PERF_KEY_H2D_BYTES (read-only): perf_run_host copies only the kept rows
    of the row scheme host -> device (PERF_KEY_HOST_SKIP, default 1); host-only."""
    W, B = 640, 2
    with kp.Plan("gaussian", W, H, 2, scheme, rate, "li", batch=B) as p:
        assert p.get("host_skip") == 1
        assert p.get("h2d_bytes") == rows * W * 4 * B
        p.set("host_skip", 0)
        assert p.get("h2d_bytes") == H * W * 4 * B
        with pytest.raises(kp.PerfError):
            p.set("h2d_bytes", 1)
