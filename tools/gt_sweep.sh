mkdir -p gpurun_out
export RUNS=4
python tools/grep_timing.py > gpurun_out/gt_base.log 2>&1
for ch in 4096 8192; do GFS_GREP_WARP=1 CHUNK=$ch python tools/grep_timing.py > gpurun_out/gt_warp_$ch.log 2>&1; done
GFS_GREP_WARP=1 CHUNK=4096 BLOCK=128 python tools/grep_timing.py > gpurun_out/gt_warp_4096_128.log 2>&1
