import ctypes, torch, os
L = ctypes.CDLL("tools/libbwprobe.so")
L.bwp_block_ms.restype = ctypes.c_float
L.bwp_block_ms.argtypes = [ctypes.c_void_p, ctypes.c_void_p, ctypes.c_longlong, ctypes.c_longlong, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_void_p]
n = 1 << 29  # 512 MiB out (8 x 4096^2 fp32)
a = torch.empty(n // 4, device="cuda"); b = torch.empty(n // 4, device="cuda")
for kn, kd in ((1, 1), (1, 2), (3, 4), (1, 4)):
    for bb in (4096, 8192, 16384):
        for br in (32, 128):
            ms = L.bwp_block_ms(a.data_ptr(), b.data_ptr(), n, 16384, bb, br, kn, kd, 16384, 1, 4, 0)
            print(f"keep {kn}/{kd} block {bb:5d} B x {br:3d} rows: {ms:.4f} ms  {(kn/kd + 1) * n / ms / 1e6:.0f} GB/s")
