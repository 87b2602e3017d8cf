"""CPU-only: the C-ABI library loads and exports every symbol include/*.h declares."""
import ctypes
import os
import re

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def declared_functions():
    names = set()
    for h in ("gpufs.h",):
        src = open(os.path.join(ROOT, "include", h)).read()
        src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
        for m in re.finditer(r"^\s*(?:const\s+)?[A-Za-z_][\w\s\*]*?\b(gfs_\w+)\s*\(", src, flags=re.M):
            names.add(m.group(1))
    return sorted(names)


def test_header_declares_the_boundary():
    names = declared_functions()
    for n in ["gfs_init", "gfs_daemon", "gfs_daemon_stop", "gfs_shutdown", "gfs_device_ctx", "gfs_stats",
              "gfs_run_gread", "gfs_run_seqread", "gfs_run_randread", "gfs_run_gwrite", "gfs_run_fileop"]:
        assert n in names


def test_library_exports_every_declared_symbol():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    from paper_conf_asplos_silbersteinfkw13_b200 import build
    build.build()
    L = ctypes.CDLL(g.LIB_PATH)
    missing = [n for n in declared_functions() if not hasattr(L, n)]
    assert not missing, missing
    g.lib()  # argtypes bind


def test_device_api_header_names():
    src = open(os.path.join(ROOT, "include", "gpufs_device.cuh")).read()
    for n in ["gopen", "gread", "gwrite", "gfsync", "gmmap", "gmunmap", "gclose", "gfstat_size", "gftruncate"]:
        assert re.search(r"__device__ inline [\w\*\s]+\b%s\(" % n, src), n


def test_config_default_without_gpu():
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    c = g.gfs_config_default()
    assert c.page_size == 64 << 10 and c.ring_slots == 4096 and c.max_batch == 32


def test_init_without_gpu_fails_loudly():
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    with pytest.raises(g.GfsError):
        g.gfs_init(g.gfs_config_default())


def test_struct_layouts_match_the_header(tmp_path):
    """ctypes mirrors of gfs_config / gfs_export_desc have the C sizes (gcc on include/gpufs.h)."""
    import ctypes
    import shutil
    import subprocess
    import paper_conf_asplos_silbersteinfkw13_b200 as g
    if not shutil.which("gcc"):
        pytest.skip("no gcc")
    src = tmp_path / "sz.c"
    src.write_text('#include <stdio.h>\n#include "gpufs.h"\nint main(void){printf("%zu %zu %zu\\n",'
                   ' sizeof(gfs_config), sizeof(gfs_export_desc), sizeof(gfs_peer)); return 0;}\n')
    exe = tmp_path / "sz"
    subprocess.check_call(["gcc", "-I", os.path.join(ROOT, "include"), str(src), "-o", str(exe)])
    cfg, desc, peer = map(int, subprocess.check_output([str(exe)]).split())
    assert ctypes.sizeof(g.gfs_config) == cfg
    assert ctypes.sizeof(g.gfs_export_desc) == desc
    assert peer == 7 * 8 + 4 * 4
