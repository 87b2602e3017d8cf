mkdir -p gpurun_out
for i in 1 2 3; do timeout 300 python bench.py --steps 5 --warmup 3 --no-hit --no-grep --no-matvec --no-c5 --no-fig4 --no-k1 --no-cpu 2>&1 | grep '^{' | python -c "
import json,sys; d=json.loads(sys.stdin.read()); print(d['value'], d['roofline']['peak'], d['clocks'])" >> gpurun_out/c2_runs.log; done
