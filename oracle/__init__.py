"""TEST INFRASTRUCTURE ONLY -- the CPU oracle of local memory-aware kernel
perforation (Maier, Cosenza, Juurlink, CGO'18).

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this module.  The
product path (``paper_conf_cgo_maiercj18_b200``) never imports it and shares
no code with it; the only common input is ``synth`` (seeded generators).

The arithmetic lives in ``kperf_oracle.c`` (plain C, fp64); this file only
marshals numpy arrays through ctypes.  Functions with no independent pin:
none -- every function is pinned by tests/test_oracle_pins.py (see DESIGN.md
"Pins").
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "liboracle.so")

APPS = {"gaussian": 0, "sobel": 1, "median": 2, "hotspot": 3, "gauss_sobel": 4, "inversion": 5}
SCHEMES = {"none": 0, "row": 1, "col": 2, "checker": 3, "stencil1": 4}
RECONS = {"nn": 0, "li": 1}
METRICS = {"mre": 0, "me": 1, "mae": 2}


class OrcParams(ctypes.Structure):
    _fields_ = [(n, ctypes.c_int) for n in
                ("app", "W", "H", "radius", "scheme", "num", "den", "recon", "granule", "tile_w", "tile_h",
                 "tblock")]


def build(force: bool = False) -> str:
    """Compile liboracle.so (gcc, -O2 -ffp-contract=off: no FMA contraction)."""
    src = os.path.join(_HERE, "kperf_oracle.c")
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(src):
        subprocess.check_call(["gcc", "-O2", "-ffp-contract=off", "-fPIC", "-shared", "-std=c99",
                               "-o", _LIB_PATH, src, "-lm"])
    return _LIB_PATH


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB_PATH)
        P = ctypes.POINTER(OrcParams)
        vp = ctypes.c_void_p
        i = ctypes.c_int
        ll = ctypes.c_longlong
        d = ctypes.c_double
        sig = {
            "orc_is_kept": (i, [P, i, i]),
            "orc_R_f32": (d, [P, vp, i, i]),
            "orc_R_u8": (i, [P, vp, i, i]),
            "orc_reconstruct_f32": (None, [P, vp, vp]),
            "orc_reconstruct_u8": (None, [P, vp, vp]),
            "orc_run_f32": (None, [P, vp, vp]),
            "orc_run_u8": (None, [P, vp, vp]),
            "orc_run_pixel_f32": (d, [P, vp, i, i]),
            "orc_run_pixel_u8": (i, [P, vp, i, i]),
            "orc_hotspot_coeffs": (None, [vp, vp, vp, vp, vp]),
            "orc_hotspot_run": (None, [P, vp, vp, i, vp]),
            "orc_hotspot_rect": (None, [P, vp, vp, i, i, i, i, i, vp]),
            "orc_hotspot_window": (None, [P, vp, vp, i, i, i, i, i]),
            "orc_error_f64": (d, [i, vp, vp, ll, vp]),
            "orc_error_f32": (d, [i, vp, vp, ll, vp]),
            "orc_error_u8": (d, [i, vp, vp, ll, vp]),
        }
        for name, (res, args) in sig.items():
            fn = getattr(L, name)
            fn.restype = res
            fn.argtypes = args
        _lib = L
    return _lib


def params(app="gaussian", W=0, H=0, radius=2, scheme="none", rate=(0, 1), recon="nn", granule=8, tile=(16, 16),
           tblock=1):
    num, den = rate
    return OrcParams(APPS[app], W, H, radius, SCHEMES[scheme], num, den, RECONS[recon], granule, tile[0], tile[1],
                     tblock)


def _ptr(a: np.ndarray):
    assert a.flags["C_CONTIGUOUS"]
    return a.ctypes.data_as(ctypes.c_void_p)


def mask(p: OrcParams) -> np.ndarray:
    L = lib()
    m = np.zeros((p.H, p.W), dtype=np.uint8)
    for y in range(p.H):
        for x in range(p.W):
            m[y, x] = L.orc_is_kept(ctypes.byref(p), x, y)
    return m


def reconstruct(p: OrcParams, img: np.ndarray) -> np.ndarray:
    L = lib()
    if img.dtype == np.uint8:
        out = np.zeros_like(img)
        L.orc_reconstruct_u8(ctypes.byref(p), _ptr(img), _ptr(out))
    else:
        img = np.ascontiguousarray(img, dtype=np.float32)
        out = np.zeros(img.shape, dtype=np.float64)
        L.orc_reconstruct_f32(ctypes.byref(p), _ptr(img), _ptr(out))
    return out


def run(p: OrcParams, img: np.ndarray) -> np.ndarray:
    """Whole-image perforated (or exact, scheme none / num 0) stencil output."""
    L = lib()
    if img.dtype == np.uint8:
        out = np.zeros_like(img)
        L.orc_run_u8(ctypes.byref(p), _ptr(img), _ptr(out))
    else:
        img = np.ascontiguousarray(img, dtype=np.float32)
        out = np.zeros(img.shape, dtype=np.float64)
        L.orc_run_f32(ctypes.byref(p), _ptr(img), _ptr(out))
    return out


def run_pixels(p: OrcParams, img: np.ndarray, xs, ys) -> np.ndarray:
    """Selected output pixels, each rebuilt from its own window (sampled checks)."""
    L = lib()
    if img.dtype == np.uint8:
        return np.array([L.orc_run_pixel_u8(ctypes.byref(p), _ptr(img), int(x), int(y))
                         for x, y in zip(xs, ys)], dtype=np.uint8)
    img = np.ascontiguousarray(img, dtype=np.float32)
    return np.array([L.orc_run_pixel_f32(ctypes.byref(p), _ptr(img), int(x), int(y))
                     for x, y in zip(xs, ys)], dtype=np.float64)


def hotspot_coeffs():
    vals = [ctypes.c_double() for _ in range(5)]
    lib().orc_hotspot_coeffs(*[ctypes.byref(v) for v in vals])
    return tuple(v.value for v in vals)


def hotspot(p: OrcParams, T0: np.ndarray, P: np.ndarray, iters: int) -> np.ndarray:
    T0 = np.ascontiguousarray(T0, dtype=np.float32)
    P = np.ascontiguousarray(P, dtype=np.float32)
    out = np.zeros(T0.shape, dtype=np.float64)
    lib().orc_hotspot_run(ctypes.byref(p), _ptr(T0), _ptr(P), iters, _ptr(out))
    return out


def hotspot_rect(p: OrcParams, T0, P, iters, x0, y0, w, h) -> np.ndarray:
    T0 = np.ascontiguousarray(T0, dtype=np.float32)
    P = np.ascontiguousarray(P, dtype=np.float32)
    out = np.zeros((h, w), dtype=np.float64)
    lib().orc_hotspot_rect(ctypes.byref(p), _ptr(T0), _ptr(P), iters, x0, y0, w, h, _ptr(out))
    return out


def hotspot_window(p: OrcParams, T: np.ndarray, P: np.ndarray, ox: int, oy: int, iters: int) -> None:
    """iters steps in place on a window (fp64 T, fp32 P) whose pixel (0,0) is global (ox, oy)"""
    assert T.dtype == np.float64 and T.flags["C_CONTIGUOUS"] and T.shape == P.shape
    P = np.ascontiguousarray(P, dtype=np.float32)
    h, w = T.shape
    lib().orc_hotspot_window(ctypes.byref(p), _ptr(T), _ptr(P), ox, oy, w, h, iters)


def error(metric: str, exact: np.ndarray, approx: np.ndarray):
    """(error value, count) of approx against exact."""
    L = lib()
    cnt = ctypes.c_longlong()
    m = METRICS[metric]
    assert exact.shape == approx.shape
    n = exact.size
    if exact.dtype == np.uint8:
        v = L.orc_error_u8(m, _ptr(exact), _ptr(np.ascontiguousarray(approx, np.uint8)), n, ctypes.byref(cnt))
    elif exact.dtype == np.float32:
        v = L.orc_error_f32(m, _ptr(exact), _ptr(np.ascontiguousarray(approx, np.float32)), n,
                            ctypes.byref(cnt))
    else:
        v = L.orc_error_f64(m, _ptr(np.ascontiguousarray(exact, np.float64)),
                            _ptr(np.ascontiguousarray(approx, np.float64)), n, ctypes.byref(cnt))
    return v, cnt.value


def default_metric(app: str) -> str:
    """Table 1: MRE everywhere except Sobel's mean error."""
    return "me" if app in ("sobel", "gauss_sobel") else "mre"
