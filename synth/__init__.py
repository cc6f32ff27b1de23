"""Seeded synthetic inputs (the only module both the oracle side and the CUDA
side use).  No method arithmetic lives here: see synth.h.

Host generation returns numpy arrays; device generation writes into caller
device pointers (torch tensors' ``data_ptr()``) on a caller stream.  Both run
the same integer functions and are bit-identical.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "libsynth.so")

FLAT, NATURAL, PATTERN = 0, 1, 2
CLASSES = {"flat": FLAT, "natural": NATURAL, "pattern": PATTERN}

# seeds of the BASELINE.json configs
SEED_C1 = 0x5EED0001
SEED_C2 = 0x5EED0010  # + class
SEED_C3 = 0x5EED0020
SEED_C4 = 0x5EED0030
SEED_C5 = 0x5EED1000  # + frame


def build(force: bool = False) -> str:
    src = os.path.join(_HERE, "synth_gen.cu")
    hdr = os.path.join(_HERE, "synth.h")
    newest = max(os.path.getmtime(src), os.path.getmtime(hdr))
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < newest:
        subprocess.check_call(["nvcc", "-O3", "-std=c++17", "-gencode", "arch=compute_100a,code=sm_100a",
                               "-Xcompiler", "-fPIC", "-shared", "-o", _LIB_PATH, src])
    return _LIB_PATH


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB_PATH)
        vp, i, u64 = ctypes.c_void_p, ctypes.c_int, ctypes.c_ulonglong
        for name, args in {
            "synth_image_f32_host": [i, u64, i, i, vp],
            "synth_image_u8_host": [i, u64, i, i, vp],
            "synth_hotspot_host": [u64, i, i, vp, vp],
            "synth_image_f32_device": [i, u64, i, i, i, vp, vp],
            "synth_image_u8_device": [i, u64, i, i, i, vp, vp],
            "synth_hotspot_device": [u64, i, i, vp, vp, vp],
            "synth_hotspot_band_device": [u64, i, i, i, i, vp, vp, vp],
        }.items():
            fn = getattr(L, name)
            fn.restype = ctypes.c_int
            fn.argtypes = args
        _lib = L
    return _lib


def _cls(c):
    return CLASSES[c] if isinstance(c, str) else int(c)


def image(cls, seed: int, W: int, H: int, dtype=np.float32) -> np.ndarray:
    out = np.zeros((H, W), dtype=dtype)
    fn = lib().synth_image_u8_host if dtype == np.uint8 else lib().synth_image_f32_host
    fn(_cls(cls), seed, W, H, out.ctypes.data_as(ctypes.c_void_p))
    return out


def hotspot(seed: int, W: int, H: int):
    T = np.zeros((H, W), dtype=np.float32)
    P = np.zeros((H, W), dtype=np.float32)
    lib().synth_hotspot_host(seed, W, H, T.ctypes.data_as(ctypes.c_void_p), P.ctypes.data_as(ctypes.c_void_p))
    return T, P


def image_device(cls, seed0: int, W: int, H: int, frames: int, ptr: int, u8: bool, stream: int = 0) -> None:
    fn = lib().synth_image_u8_device if u8 else lib().synth_image_f32_device
    rc = fn(_cls(cls), seed0, W, H, frames, ptr, stream)
    if rc != 0:
        raise RuntimeError(f"synth device generation failed (cuda error {rc})")


def hotspot_device(seed: int, W: int, H: int, t_ptr: int, p_ptr: int, stream: int = 0) -> None:
    rc = lib().synth_hotspot_device(seed, W, H, t_ptr, p_ptr, stream)
    if rc != 0:
        raise RuntimeError(f"synth device generation failed (cuda error {rc})")


def hotspot_band_device(seed: int, W: int, H: int, y0: int, h: int, t_ptr: int, p_ptr: int,
                        stream: int = 0) -> None:
    rc = lib().synth_hotspot_band_device(seed, W, H, y0, h, t_ptr, p_ptr, stream)
    if rc != 0:
        raise RuntimeError(f"synth device generation failed (cuda error {rc})")
