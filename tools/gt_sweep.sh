# C4 grep timing sweep over (chunk, block) for the block scan (and optionally GFS_GREP_WARP=1)
mkdir -p gpurun_out
export RUNS=4
for cb in 32768:256 32768:128 16384:256 16384:128 8192:128 65536:256; do
  ch=${cb%%:*}; bl=${cb##*:}
  CHUNK=$ch BLOCK=$bl python tools/grep_timing.py 2>&1 | tail -1 >> gpurun_out/gt_sweep.log
done
