mkdir -p gpurun_out
{
echo "nproc: $(nproc)"; python -c "import os; print('affinity', sorted(os.sched_getaffinity(0)))"
ls /sys/devices/system/node/ | grep node
for n in /sys/devices/system/node/node*; do echo "$n: $(cat $n/cpulist)"; done
bus=$(nvidia-smi --query-gpu=pci.bus_id --format=csv,noheader | head -1 | tr 'A-F' 'a-f' | sed 's/^0000//')
echo "gpu bus $bus"; cat /sys/bus/pci/devices/0000${bus#0000}/numa_node 2>/dev/null || cat /sys/bus/pci/devices/${bus}/numa_node 2>/dev/null
ls /sys/bus/pci/devices/ | grep -i "${bus: -7}" | head
lscpu | grep -iE "socket|numa|model name"
} > gpurun_out/numa.log 2>&1
