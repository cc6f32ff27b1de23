#!/bin/bash
# One GPU pass of the round's measurement evidence (run under gpurun from the
# repo root); everything lands in gpurun_out/prof/.  Bench numbers are NOT
# taken under ncu: the benches run first, ncu passes after.
set -u
O=gpurun_out/prof
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.log 2>&1
# --- benches (driver contract lines) ---
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
for c in C1 C3 C5; do python bench.py --config $c > $O/bench_$c.json 2> $O/bench_$c.err; done
python bench.py --config C4 --steps 5 > $O/bench_C4.json 2> $O/bench_C4.err
python bench.py --config C4 --steps 5 --tblock 8 --no-variants --no-cpu > $O/bench_C4_tb8.json 2> $O/bench_C4_tb8.err
python bench.py --impl reference --steps 3 --warmup 3 > $O/bench_C2_reference.json 2> $O/bench_C2_reference.err
# --- ncu: launch list of the default bench (shares, not times) ---
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches_bench_c2.csv \
  python bench.py --steps 2 --warmup 3 --no-variants --no-cpu > $O/launches_bench_c2.log 2>&1
# --- ncu --set full: headline + exact (8 x 4096^2, one measured launch each) ---
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 1 -c 1 -f -o $O/ncu_full_headline \
  python tools/ncu_driver.py --variants headline --batch 8 > /dev/null 2>&1
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 3 -c 1 -f -o $O/ncu_full_exact \
  python tools/ncu_driver.py --variants headline --batch 8 > /dev/null 2>&1
# --- ncu: DRAM bytes / time / instructions of every C2 variant and C1/C3/C5 ---
M=dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum,smsp__inst_executed.sum,sm__warps_active.avg.pct_of_peak_sustained_active
for v in all c1 c3 c5; do
  ncu --metrics $M --clock-control none -k regex:perf_kernel --csv --log-file $O/ncu_variants_$v.csv \
    python tools/ncu_driver.py --variants $v --batch 2 > $O/ncu_variants_$v.log 2>&1
done
# --- ncu: temporally blocked Hotspot (TBLOCK 8, 8192^2): row 1/2 LI and exact ---
ncu --set full --import-source on --clock-control none -k regex:hotspot_tb -s 1 -c 1 -f -o $O/ncu_full_tb8_row \
  python tools/ncu_hotspot_tb.py 8 > /dev/null 2>&1
ncu --set full --import-source on --clock-control none -k regex:hotspot_tb -s 3 -c 1 -f -o $O/ncu_full_tb8_exact \
  python tools/ncu_hotspot_tb.py 8 > /dev/null 2>&1
ls -la $O
