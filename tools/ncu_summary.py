"""One-kernel summary of an ncu --set full report (raw page) -> text lines."""
import csv
import io
import subprocess
import sys

KEYS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "smsp__inst_executed.sum",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "launch__registers_per_thread", "launch__occupancy_limit_registers", "launch__occupancy_limit_shared_mem",
        "launch__grid_size", "launch__block_size", "launch__shared_mem_per_block_dynamic",
        "sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active",
        "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active",
        "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum", "lts__t_bytes.sum"]


def summary(rep, idx=0):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units, vals = rows[0], rows[1], rows[2 + idx]
    v, u = dict(zip(hdr, vals)), dict(zip(hdr, units))
    lines = [f"kernel: {v.get('Kernel Name', '')}"]
    for k in KEYS:
        if k in v:
            lines.append(f"  {k:62s} {v[k]} {u.get(k, '')}")
    st = [(h, float(x)) for h, x in v.items()
          if h.startswith("smsp__average_warps_issue_stalled") and x.replace(".", "", 1).isdigit()]
    lines.append("  top stall reasons (warps per issued instruction):")
    for h, x in sorted(st, key=lambda t: -t[1])[:6]:
        lines.append(f"    {x:7.3f} {h[34:]}")
    return "\n".join(lines)


if __name__ == "__main__":
    print(summary(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 0))
