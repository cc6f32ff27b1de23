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
