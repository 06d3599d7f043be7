#!/bin/bash
# On the GPU box: the round's ncu evidence for the given configs (default c3 c2 c4_z1.5 c5_gpu).
#   launch list : every launch of our kernels in `bench.py --steps 2 --warmup 1` (duration, DRAM bytes)
#   full set    : one warm join of tools/prof_one.py, all five kernels, plus L2 write sectors per
#                 request and shared-atomic counts
# Summarised on the box (tools/profile_summary.py -> gpurun_out/ev/profiles/): gpurun copies back
# at most 64 MiB, so the .ncu-rep files are deleted after summarising (KEEP_REP=1 keeps them).
mkdir -p gpurun_out/ev/profiles
for c in ${@:-c3 c2 c4_z1.5 c5_gpu}; do
  timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    -k regex:^k_ --csv --log-file gpurun_out/ev/launches_$c.csv \
    python bench.py --config $c --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/ev/launches_$c.log 2>&1
  timeout 900 ncu --set full --import-source on --clock-control none \
    --metrics lts__t_sectors_op_write.sum,lts__t_requests_op_write.sum,smsp__sass_inst_executed_op_shared_atom.sum \
    -k regex:^k_ --launch-skip 5 --launch-count 5 -o gpurun_out/ev/full_$c -f \
    python tools/prof_one.py $c > gpurun_out/ev/full_$c.log 2>&1
  python tools/profile_summary.py r02 gpurun_out/ev/launches_$c.csv gpurun_out/ev/full_$c.ncu-rep $c \
    --outdir gpurun_out/ev/profiles > gpurun_out/ev/summary_$c.log 2>&1
  python tools/src_hot.py gpurun_out/ev/full_$c.ncu-rep k_join 30 > gpurun_out/ev/profiles/r02_src_join_$c.txt 2>&1
  python tools/sass_smem.py gpurun_out/ev/full_$c.ncu-rep "k_pass_ws" 0 > gpurun_out/ev/profiles/r02_smem_pass_$c.txt 2>&1
  [ -n "$KEEP_REP" ] || rm -f gpurun_out/ev/full_$c.ncu-rep
done
