"""Summarise `nvcc -Xptxas -v` output: kernel -> registers, spills, stack."""
import re
import subprocess
import sys

ROOT = __file__.rsplit("/tools/", 1)[0]


def summary(src):
    cmd = ["nvcc", "-gencode", "arch=compute_100a,code=sm_100a", "-std=c++17", "-O3", "-Xptxas", "-v",
           "-Xcompiler", "-fPIC", "-c", src, "-o", "/dev/null"]
    out = subprocess.run(cmd, capture_output=True, text=True).stderr
    cur = None
    rows = []
    for line in out.splitlines():
        m = re.search(r"Compiling entry function '(\S+)'", line)
        if m:
            cur = m.group(1)
            continue
        m = re.search(r"(\d+) bytes stack frame, (\d+) bytes spill stores, (\d+) bytes spill loads", line)
        if m and cur:
            stack, ss, sl = map(int, m.groups())
            continue
        m = re.search(r"Used (\d+) registers", line)
        if m and cur:
            d = re.sub(r"_ZN2kp11perf_kernelINS_\d+", "", cur)
            rows.append((d[:40], int(m.group(1)), ss, sl, stack))
            cur = None
    return rows


if __name__ == "__main__":
    for src in sys.argv[1:]:
        for r in summary(src):
            print(f"{src.split('/')[-1]:14s} {r[0]:40s} regs {r[1]:4d} spill {r[2]}/{r[3]} stack {r[4]}")
