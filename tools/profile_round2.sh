#!/bin/bash
# One GPU pass of round 2's measurement evidence (run under gpurun from the repo
# root); everything lands in gpurun_out/r02/.  Bench numbers are never taken
# under ncu: the ncu passes are separate processes.
set -u
O=gpurun_out/r02
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.log 2>&1
# per-launch ncu counters of every config's headline + exact kernel (bench reads them)
python tools/ncu_traffic.py > $O/ncu_traffic.log 2>&1; cp profiles/ncu_traffic.json $O/
# benches (driver contract lines)
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
for c in C1 C3 C5; do python bench.py --config $c > $O/bench_$c.json 2> $O/bench_$c.err; done
python bench.py --config C4 --steps 5 > $O/bench_C4.json 2> $O/bench_C4.err
python bench.py --sweep > $O/sweep_c2.json 2> $O/sweep_c2.err
python bench.py --impl reference --steps 3 --warmup 3 > $O/bench_C2_reference.json 2> $O/bench_C2_reference.err
# launch list of the default bench (shares, not times)
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches_bench_c2.csv \
  python bench.py --steps 2 --warmup 3 --no-variants --no-cpu > $O/launches_bench_c2.log 2>&1
# ncu --set full: headline + exact (8 x 4096^2, one measured launch each), C3 and C5 headlines
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 1 -c 1 -f -o $O/ncu_full_headline \
  python tools/ncu_driver.py --variants headline --batch 8 > /dev/null 2>&1
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 3 -c 1 -f -o $O/ncu_full_exact \
  python tools/ncu_driver.py --variants headline --batch 8 > /dev/null 2>&1
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 3 -c 1 -f -o $O/ncu_full_c3_col12 \
  python tools/ncu_driver.py --variants c3 --batch 4 > /dev/null 2>&1
ncu --set full --import-source on --clock-control none -k regex:perf_kernel -s 3 -c 1 -f -o $O/ncu_full_c5_row12 \
  python tools/ncu_driver.py --variants c5 --batch 16 > /dev/null 2>&1
# DRAM bytes / time / instructions of every C2 variant (128-B and 1-px cells) and C1/C3/C5
M=dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum,smsp__inst_executed.sum,sm__warps_active.avg.pct_of_peak_sustained_active
for v in all c1 c3all c5; do
  ncu --metrics $M --clock-control none -k regex:perf_kernel --csv --log-file $O/ncu_variants_$v.csv \
    python tools/ncu_driver.py --variants $v --batch 2 > $O/ncu_variants_$v.log 2>&1
done
ncu --metrics $M --clock-control none -k regex:perf_kernel --csv --log-file $O/ncu_variants_all_g1px.csv \
  python tools/ncu_driver.py --variants all --batch 2 --gran 4 > $O/ncu_variants_all_g1px.log 2>&1
# sanitizers: compute-sanitizer is closed on the GPU pool since round 2b (runs
# under it left GPUs needing a reset); the committed round-2 logs
# (profiles/r02/sanitizer_*.log) predate the 2b kernel changes
ls -la $O
