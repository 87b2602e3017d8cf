mkdir -p gpurun_out
for v in ${VARS:-C B D C B D}; do
  cp variants/lib$v.so paper_conf_asplos_silbersteinfkw13_b200/libgpufs.so
  timeout 400 python bench.py --steps 3 --warmup 3 --no-fig4 --no-c5 --no-k1 --no-cpu 2>/dev/null | grep '^{' | python -c "
import json,sys; d=json.loads(sys.stdin.read())
print('$v', 'C2', d['value'], 'K4', d['hit']['GBps'], 'raw', d['hit']['raw_GBps'], 'C4warm', d['grep']['warm']['ms'], 'C3', d['matvec']['GBps'], 'h2d', d['roofline']['peak'])" >> gpurun_out/variants.log 2>&1
done
