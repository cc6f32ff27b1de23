"""Count local-memory (LDL/STL) instructions in a kernel's SASS, split into the
kernel body and the functions it CALLs (e.g. the noinline generic consumer).
usage: sass_local.py file.o|lib.so mangled-kernel-name"""
import re
import subprocess
import sys

out = subprocess.run(["cuobjdump", "-sass", "-fun", sys.argv[2], sys.argv[1]], capture_output=True, text=True).stdout
ins = [(int(m.group(1), 16), m.group(2)) for m in re.finditer(r"/\*([0-9a-f]{4,})\*/\s+([^;]*);", out)]
calls = sorted({int(m, 16) for _, t in ins for m in re.findall(r"CALL\.\S+\s+0x([0-9a-f]+)", t)})
cut = calls[0] if calls else 1 << 60
body = [t for a, t in ins if a < cut]
rest = [t for a, t in ins if a >= cut]
loc = lambda xs: sum(1 for t in xs if re.search(r"\b(LDL|STL)", t))  # noqa: E731
print(f"body: {len(body)} instr, {loc(body)} LDL/STL; called functions (from {cut:#x}): {len(rest)} instr, {loc(rest)} LDL/STL")
