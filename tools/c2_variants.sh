# C2 headline only, alternating library variants (variants/lib$v.so), same box
mkdir -p gpurun_out
for v in ${VARS:-S M S M S M}; do
  cp variants/lib$v.so paper_conf_asplos_silbersteinfkw13_b200/libgpufs.so
  timeout 300 python bench.py --steps 5 --warmup 3 --no-hit --no-grep --no-matvec --no-c5 --no-fig4 --no-k1 --no-cpu 2>/dev/null \
    | grep '^{' | python -c "
import json,sys; d=json.loads(sys.stdin.read()); print('$v', d['value'], d['roofline']['peak'], d['e2e']['value'])" >> gpurun_out/c2_variants.log
done
