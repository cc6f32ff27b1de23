"""B200-native hot path of local memory-aware kernel perforation
(Maier, Cosenza, Juurlink, CGO'18).

A thin ctypes binding over the C ABI in ``include/kperf.h`` (libkperf.so,
sm_100a).  Functions keep the C names; the only work done here is argument
marshalling (tensor -> device pointer, stream -> handle, status -> exception).
Every step of the path runs in the CUDA kernels of libkperf.so; there is no
CPU fallback: if the library is missing or the device is not an sm_100 GPU,
calls raise.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("KPERF_LIB", os.path.join(_HERE, "libkperf.so"))  # override: experiment builds

# enums (mirror include/kperf.h)
APP = {"gaussian": 0, "sobel": 1, "median": 2, "hotspot": 3, "gauss_sobel": 4, "inversion": 5}
SCHEME = {"none": 0, "row": 1, "col": 2, "checker": 3, "stencil1": 4}
RECON = {"nn": 0, "li": 1, "linear": 1}
METRIC = {"mre": 0, "me": 1, "mae": 2}
KEY = {"batch": 1, "iters": 2, "granule_bytes": 3, "global_h": 4, "band_y0": 5, "tile_w": 6, "tile_h": 7,
       "metric": 8, "loader": 9, "ring": 10, "halo_rows": 11, "tile1_w": 12, "tile1_h": 13, "producer": 14,
       "tblock": 15, "p2p": 16, "chk_compact": 17, "overlap": 18, "graph": 19, "exchange": 20, "fold": 21,
       "host_skip": 22, "h2d_bytes": 23}
STATUS = {0: "PERF_OK", 1: "PERF_ERR_INVALID_ARG", 2: "PERF_ERR_UNSUPPORTED", 3: "PERF_ERR_CUDA",
          4: "PERF_ERR_NCCL", 5: "PERF_ERR_OOM"}

# exported symbols of include/kperf.h (tests check the library exports all of them)
SYMBOLS = ("perf_plan", "perf_plan_set", "perf_plan_get", "perf_run", "perf_run_host", "perf_run_hotspot",
           "perf_run_hotspot_bands_local", "perf_error", "perf_error_sums", "perf_error_finish",
           "perf_error_allreduce", "perf_band_halo", "perf_run_band", "perf_comm_init", "perf_comm_unique_id",
           "perf_p2p_export", "perf_p2p_attach", "perf_destroy", "perf_last_error", "perf_version")


class PerfRate(ctypes.Structure):
    _fields_ = [("num", ctypes.c_int), ("den", ctypes.c_int)]


class PerfHaloPlan(ctypes.Structure):
    _fields_ = [(n, ctypes.c_int) for n in ("halo_rows", "buf_rows", "up_rank", "down_rank", "send_up_row",
                                            "recv_up_row", "send_down_row", "recv_down_row")]


class PerfError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS.get(status, status)}: {msg}")
        self.status = status


_lib = None


def lib():
    """Load libkperf.so (raises if it was not built)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} missing: run __graft_entry__.build() (no CPU fallback exists)")
        L = ctypes.CDLL(LIB_PATH)
        vp, i, ll = ctypes.c_void_p, ctypes.c_int, ctypes.c_longlong
        sig = {
            "perf_plan": [ctypes.POINTER(vp), i, i, i, i, i, PerfRate, i],
            "perf_plan_set": [vp, i, ll],
            "perf_plan_get": [vp, i, ctypes.POINTER(ll)],
            "perf_run": [vp, vp, vp, vp],
            "perf_run_host": [vp, vp, vp, vp],
            "perf_run_hotspot": [vp, vp, vp, vp, vp],
            "perf_run_hotspot_bands_local": [ctypes.POINTER(vp), i, vp, vp, vp, vp],
            "perf_error": [vp, vp, vp, vp, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ll)],
            "perf_error_sums": [vp, vp, vp, vp, ctypes.POINTER(ctypes.c_double)],
            "perf_error_finish": [vp, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ctypes.c_double),
                                  ctypes.POINTER(ll)],
            "perf_error_allreduce": [vp, vp, vp, vp, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ll)],
            "perf_band_halo": [vp, i, i, ctypes.POINTER(PerfHaloPlan)],
            "perf_run_band": [vp, vp, vp, vp],
            "perf_comm_init": [vp, vp, i, i],
            "perf_comm_unique_id": [vp],
            "perf_p2p_export": [vp, vp],
            "perf_p2p_attach": [vp, vp, vp],
            "perf_destroy": [vp],
        }
        for name, args in sig.items():
            fn = getattr(L, name)
            fn.argtypes = args
            fn.restype = ctypes.c_int
        L.perf_last_error.restype = ctypes.c_char_p
        L.perf_last_error.argtypes = []
        L.perf_version.restype = ctypes.c_char_p
        L.perf_version.argtypes = []
        _lib = L
    return _lib


def _check(status: int):
    if status != 0:
        raise PerfError(status, lib().perf_last_error().decode())


def _ptr(x) -> int:
    if x is None:
        return None
    if isinstance(x, int):
        return x
    if hasattr(x, "data_ptr"):  # torch tensor
        return x.data_ptr()
    if hasattr(x, "ctypes"):    # numpy array (host buffers for perf_run_host)
        return x.ctypes.data
    raise TypeError(f"cannot take a pointer of {type(x)}")


def _check_buf(x, app, numel, device, name):
    """Argument checks before a pointer crosses the C ABI: dense, the plan's
    element type, on the right side of the bus, exactly W*H*BATCH elements
    (the ABI takes bare pointers and cannot check any of this)."""
    if x is None or isinstance(x, int):
        return  # raw pointers: the caller's contract (include/kperf.h)
    want = "uint8" if app == "median" else "float32"
    if hasattr(x, "data_ptr"):  # torch tensor
        if not x.is_contiguous():
            raise ValueError(f"{name}: tensor must be contiguous")
        if str(x.dtype).replace("torch.", "") != want:
            raise TypeError(f"{name}: dtype {x.dtype}, plan needs {want}")
        if (x.device.type == "cuda") != device:
            raise ValueError(f"{name}: tensor on {x.device}, expected a {'cuda' if device else 'host'} tensor")
        n = x.numel()
    elif hasattr(x, "ctypes"):  # numpy array: host memory only
        if device:
            raise ValueError(f"{name}: numpy array passed where a device buffer is needed")
        if not x.flags["C_CONTIGUOUS"]:
            raise ValueError(f"{name}: array must be C-contiguous")
        if str(x.dtype) != want:
            raise TypeError(f"{name}: dtype {x.dtype}, plan needs {want}")
        n = x.size
    else:
        raise TypeError(f"{name}: cannot take a pointer of {type(x)}")
    if n != numel:
        raise ValueError(f"{name}: {n} elements, plan needs W*H*BATCH = {numel}")


def _stream(stream) -> int:
    if stream is None:
        import torch
        return torch.cuda.current_stream().cuda_stream
    if isinstance(stream, int):
        return stream
    return stream.cuda_stream


def _enum(table, v):
    return table[v] if isinstance(v, str) else int(v)


def perf_version() -> str:
    return lib().perf_version().decode()


def perf_plan(app, W: int, H: int, radius: int, scheme="none", rate=(0, 1), recon="nn") -> int:
    h = ctypes.c_void_p()
    _check(lib().perf_plan(ctypes.byref(h), _enum(APP, app), W, H, radius, _enum(SCHEME, scheme),
                           PerfRate(*rate), _enum(RECON, recon)))
    return h.value


def perf_plan_set(plan: int, key, value: int) -> None:
    _check(lib().perf_plan_set(plan, _enum(KEY, key), int(value)))


def perf_plan_get(plan: int, key) -> int:
    v = ctypes.c_longlong()
    _check(lib().perf_plan_get(plan, _enum(KEY, key), ctypes.byref(v)))
    return v.value


def perf_run(plan: int, inp, out, stream=None) -> None:
    _check(lib().perf_run(plan, _ptr(inp), _ptr(out), _stream(stream)))


def perf_run_host(plan: int, host_in, host_out, stream=None) -> None:
    _check(lib().perf_run_host(plan, _ptr(host_in), _ptr(host_out), _stream(stream)))


def perf_run_hotspot(plan: int, temp_in, power, temp_out, stream=None) -> None:
    _check(lib().perf_run_hotspot(plan, _ptr(temp_in), _ptr(power), _ptr(temp_out), _stream(stream)))


def perf_run_hotspot_bands_local(plans, temp_in, power, temp_out, stream=None) -> None:
    arr = (ctypes.c_void_p * len(plans))(*plans)
    _check(lib().perf_run_hotspot_bands_local(arr, len(plans), _ptr(temp_in), _ptr(power), _ptr(temp_out),
                                              _stream(stream)))


def perf_error(plan: int, exact, approx, stream=None):
    v = ctypes.c_double()
    c = ctypes.c_longlong()
    _check(lib().perf_error(plan, _ptr(exact), _ptr(approx), _stream(stream), ctypes.byref(v), ctypes.byref(c)))
    return v.value, c.value


def perf_error_sums(plan: int, exact, approx, stream=None):
    """(sum of terms, sum |e|, count) -- shard sums add elementwise"""
    h = (ctypes.c_double * 3)()
    _check(lib().perf_error_sums(plan, _ptr(exact), _ptr(approx), _stream(stream), h))
    return tuple(h)


def perf_error_finish(plan: int, sums):
    """host only: the plan's metric from (summed) partial sums"""
    h = (ctypes.c_double * 3)(*[float(v) for v in sums])
    v = ctypes.c_double()
    c = ctypes.c_longlong()
    _check(lib().perf_error_finish(plan, h, ctypes.byref(v), ctypes.byref(c)))
    return v.value, c.value


def perf_error_allreduce(plan: int, exact, approx, stream=None):
    v = ctypes.c_double()
    c = ctypes.c_longlong()
    _check(lib().perf_error_allreduce(plan, _ptr(exact), _ptr(approx), _stream(stream), ctypes.byref(v),
                                      ctypes.byref(c)))
    return v.value, c.value


def perf_band_halo(plan: int, rank: int, nranks: int) -> dict:
    """host only: the band buffer geometry and halo rows exchanged with each neighbour"""
    h = PerfHaloPlan()
    _check(lib().perf_band_halo(plan, rank, nranks, ctypes.byref(h)))
    return {n: getattr(h, n) for n, _ in PerfHaloPlan._fields_}


def perf_run_band(plan: int, in_band, out, stream=None) -> None:
    _check(lib().perf_run_band(plan, _ptr(in_band), _ptr(out), _stream(stream)))


def perf_comm_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    _check(lib().perf_comm_unique_id(buf))
    return buf.raw


def perf_comm_init(plan: int, unique_id: bytes, rank: int, nranks: int) -> None:
    buf = ctypes.create_string_buffer(bytes(unique_id), 128)
    _check(lib().perf_comm_init(plan, buf, rank, nranks))


def perf_p2p_export(plan: int) -> bytes:
    buf = ctypes.create_string_buffer(128)
    _check(lib().perf_p2p_export(plan, buf))
    return buf.raw


def perf_p2p_attach(plan: int, up, down) -> None:
    ub = ctypes.create_string_buffer(bytes(up), 128) if up is not None else None
    db = ctypes.create_string_buffer(bytes(down), 128) if down is not None else None
    _check(lib().perf_p2p_attach(plan, ub, db))


def perf_destroy(plan: int) -> None:
    _check(lib().perf_destroy(plan))


def band_cuts(H: int, nranks: int):
    """Row bands of a sharded Hotspot grid: rank k owns rows [cuts[k], cuts[k+1])."""
    if nranks < 1 or H < nranks:
        raise ValueError("need 1 <= nranks <= H")
    return [H * k // nranks for k in range(nranks + 1)]


class Plan:
    """Owning wrapper: ``with Plan("gaussian", W, H, 2, "row", (1, 2), "li") as p: p.run(x, y)``."""

    def __init__(self, app, W, H, radius, scheme="none", rate=(0, 1), recon="nn", **keys):
        self.app, self.W, self.H = app, W, H
        self.handle = perf_plan(app, W, H, radius, scheme, rate, recon)
        for k, v in keys.items():
            perf_plan_set(self.handle, k, v)

    def set(self, key, value):
        perf_plan_set(self.handle, key, value)
        return self

    def get(self, key):
        return perf_plan_get(self.handle, key)

    def _elems(self):
        return self.W * self.H * (1 if self.app == "hotspot" else self.get("batch"))

    def run(self, inp, out, stream=None):
        n = self._elems()
        _check_buf(inp, self.app, n, device=True, name="in")
        _check_buf(out, self.app, n, device=True, name="out")
        perf_run(self.handle, inp, out, stream)

    def run_host(self, host_in, host_out, stream=None):
        n = self._elems()
        _check_buf(host_in, self.app, n, device=False, name="host_in")
        _check_buf(host_out, self.app, n, device=False, name="host_out")
        perf_run_host(self.handle, host_in, host_out, stream)

    def hotspot(self, temp_in, power, temp_out, stream=None):
        n = self._elems()
        for b, nm in ((temp_in, "temp_in"), (power, "power"), (temp_out, "temp_out")):
            _check_buf(b, "hotspot", n, device=True, name=nm)
        perf_run_hotspot(self.handle, temp_in, power, temp_out, stream)

    def error(self, exact, approx, stream=None):
        n = self._elems()
        _check_buf(exact, self.app, n, device=True, name="exact")
        _check_buf(approx, self.app, n, device=True, name="approx")
        return perf_error(self.handle, exact, approx, stream)

    def close(self):
        if self.handle:
            perf_destroy(self.handle)
            self.handle = None

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass
