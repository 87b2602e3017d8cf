import json, os, sys, tempfile
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import gen
import paper_conf_asplos_silbersteinfkw13_b200 as g
g.build.build()
d = json.load(open("tests/golden/grep_hand.json"))
root = tempfile.mkdtemp(dir="/dev/shm")
paths = []
for i, hx in enumerate(d["files_hex"]):
    p = os.path.join(root, f"h{i}.txt"); open(p, "wb").write(bytes.fromhex(hx)); paths.append(p)
gen.write_dict(os.path.join(root, "d.bin"), [w.encode() for w in d["words"]])
gen.write_list(os.path.join(root, "l.txt"), paths)
chunk = int(sys.argv[1]) if len(sys.argv) > 1 else 16
with g.GpuFS(cache_bytes=64 * 4096, page_size=4096, timeout_ms=10000, daemon_threads=2) as fs:
    out = fs.grep(os.path.join(root, "d.bin"), os.path.join(root, "l.txt"), hits=True, chunk=chunk, grid=8)
    print("summary", out["summary"])
    print("dev", fs.stats())
    print("host", fs.host_stats())
    print("info", fs.info())
    print("records ok", out["records"].tolist() == d["expected_records"])
