#!/bin/bash
# Profiles for profiles/ (run on the GPU box via gpurun). Kernels that post
# RPCs cannot be kernel-replayed (the host side is not replayed), so the
# full-set captures target warm kernels with files pinned open.
set -x
mkdir -p gpurun_out
# 1. every launch of a short bench run with its device time (single pass, no replay)
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
  python bench.py --steps 2 --warmup 1 --file-gib 2 --cache-gib 1 --grep-files 3000 --grep-mib 50 --no-cpu \
  > gpurun_out/bench_under_ncu.log 2>&1
# 2. K4 cache-hit kernel, full set
HIT_GRID=1184 HIT_BLOCK=128 HIT_CALLS=256 timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_randread -s 4 -c 2 \
  -o gpurun_out/prof_hit python tools/prof_hit.py > gpurun_out/ncu_hit.log 2>&1
# 3. warm grep scan kernel (second launch), full set
C4_FILES=30000 C4_MIB=500 timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_grep_scan -s 1 -c 1 \
  -o gpurun_out/prof_grep python tools/debug_c4.py > gpurun_out/ncu_grep.log 2>&1
ls -la gpurun_out
