"""CPU-only checks of the boundary: libdock.so builds for sm_100a, loads, and exports every
symbol include/dock.h declares; the binding fails loudly without the library; no compute."""
import ctypes
import os
import re

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    from paper_conf_ipps_sukhwanih10_b200 import build
    build.build_native()
    from paper_conf_ipps_sukhwanih10_b200 import _native
    return _native.lib()


def _header_functions():
    import glob
    src = "".join(open(h).read() for h in sorted(glob.glob(os.path.join(ROOT, "include", "*.h"))))
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(dock_[a-z_]+)\s*\(", src)))


def test_header_symbols_exported(lib):
    names = _header_functions()
    assert "dock_init" in names and "dock_probe_batch" in names
    for n in names:
        assert hasattr(lib, n), f"libdock.so does not export {n}"
    from paper_conf_ipps_sukhwanih10_b200 import _native
    assert sorted(_native.EXPORTS) == names


def test_status_strings(lib):
    for code, name in [(0, b"DOCK_OK"), (-1, b"DOCK_E_INVALID_ARG"), (-3, b"DOCK_E_PROBE_OUTSIDE_GRID"),
                       (-4, b"DOCK_E_BAD_ROTATION"), (-5, b"DOCK_E_CUDA")]:
        assert lib.dock_status_string(code) == name


def test_null_arguments_rejected_without_gpu(lib):
    out = ctypes.c_void_p()
    assert lib.dock_init(None, None, None, ctypes.byref(out)) == -1
    assert lib.dock_probe_batch(None, None, 0, None, 0, 0, 0, 1, 0, None) == -1
    lib.dock_destroy(None)


def test_struct_layouts():
    from paper_conf_ipps_sukhwanih10_b200 import _native as N
    assert ctypes.sizeof(N.dock_pose) == 16
    assert ctypes.sizeof(N.dock_probe_desc) == 24
    assert ctypes.sizeof(N.dock_grid_desc) == 40


def test_struct_layouts_match_header(tmp_path):
    """Every ctypes struct of the binding has the sizes and field offsets that include/dock.h gives a
    C compiler (catches a field whose type changed on one side only, e.g. the spacing's width)."""
    import shutil
    import subprocess
    from paper_conf_ipps_sukhwanih10_b200 import _native as N
    cc = shutil.which("gcc") or shutil.which("cc")
    if not cc:
        pytest.skip("no C compiler")
    structs = {"dock_pose": N.dock_pose, "dock_grid_desc": N.dock_grid_desc,
               "dock_probe_desc": N.dock_probe_desc, "dock_info": N.dock_info, "dock_em_desc": N.dock_em_desc,
               "dock_em_params": N.dock_em_params}
    lines = ['#include <stdio.h>', '#include <stddef.h>', '#include "dock.h"', '#include "dock_em.h"',
             "int main(void) {"]
    for name, cls in structs.items():
        lines.append(f'printf("{name} size %zu\\n", sizeof({name}));')
        for f, _ in cls._fields_:
            lines.append(f'printf("{name} {f} %zu\\n", offsetof({name}, {f}));')
            lines.append(f'printf("{name} {f}.size %zu\\n", sizeof((({name}*)0)->{f}));')
    lines.append("return 0; }")
    src = tmp_path / "layout.c"
    src.write_text("\n".join(lines))
    exe = tmp_path / "layout"
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    subprocess.check_call([cc, "-std=c99", "-I", os.path.join(root, "include"), "-o", str(exe), str(src)])
    got = {}
    for line in subprocess.check_output([str(exe)], text=True).splitlines():
        a, b, c = line.split()
        got[(a, b)] = int(c)
    for name, cls in structs.items():
        assert got[(name, "size")] == ctypes.sizeof(cls), name
        for f, _ in cls._fields_:
            assert got[(name, f)] == getattr(cls, f).offset, f"{name}.{f}"
            assert got[(name, f + ".size")] == getattr(cls, f).size, f"{name}.{f} width"


def test_sass_is_sm100a_with_tma():
    """The hot kernel is compiled for sm_100a and issues TMA (UTMALDG) + bulk copies (UBLKCP)."""
    import shutil
    import subprocess
    from paper_conf_ipps_sukhwanih10_b200 import build
    lib_path = build.build_native()
    cuobjdump = shutil.which("cuobjdump") or "/usr/local/cuda/bin/cuobjdump"
    if not os.path.exists(cuobjdump) and not shutil.which("cuobjdump"):
        pytest.skip("cuobjdump not available")
    out = subprocess.run([cuobjdump, "-sass", lib_path], capture_output=True, text=True).stdout
    assert "sm_100a" in out
    assert "UTMALDG" in out and "UBLKCP" in out and "FFMA" in out


def test_missing_library_fails_loudly(monkeypatch, tmp_path):
    from paper_conf_ipps_sukhwanih10_b200 import _native
    monkeypatch.setattr(_native, "_lib", None)
    monkeypatch.setattr(_native, "LIB_PATH", str(tmp_path / "nope.so"))
    with pytest.raises(ImportError):
        _native.lib()


def test_sass_has_tcgen05_mma():
    """The tensor-core engine really issues tcgen05.mma (UTCHMMA) and its commit barriers (UTCBAR)."""
    import shutil
    import subprocess
    from paper_conf_ipps_sukhwanih10_b200 import build
    lib_path = build.build_native()
    cuobjdump = shutil.which("cuobjdump") or "/usr/local/cuda/bin/cuobjdump"
    if not os.path.exists(cuobjdump) and not shutil.which("cuobjdump"):
        pytest.skip("cuobjdump not available")
    out = subprocess.run([cuobjdump, "-sass", lib_path], capture_output=True, text=True).stdout
    assert "UTCHMMA" in out and "UTCBAR" in out


def test_product_package_never_reaches_the_oracle():
    """The oracle is test infrastructure: no module of the product package imports or names it,
    and bench.py touches it only in its cpu_baseline / reference-arm helpers."""
    import ast
    pkg = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                       "paper_conf_ipps_sukhwanih10_b200")
    for root, _, files in os.walk(pkg):
        for f in files:
            if not f.endswith((".py", ".cu", ".cuh", ".h", ".c", ".cpp")):
                continue
            src = open(os.path.join(root, f), encoding="utf-8").read()
            if f.endswith(".py"):
                for node in ast.walk(ast.parse(src)):
                    if isinstance(node, ast.Import):
                        assert not any(a.name.split(".")[0] == "oracle" for a in node.names), f
                    if isinstance(node, ast.ImportFrom):
                        assert (node.module or "").split(".")[0] != "oracle", f
            else:
                assert "dock_oracle" not in src and "liboracle" not in src, f
    bench = os.path.join(os.path.dirname(pkg), "bench.py")
    tree = ast.parse(open(bench, encoding="utf-8").read())
    users = set()
    for fn in [n for n in ast.walk(tree) if isinstance(n, ast.FunctionDef)]:
        for node in ast.walk(fn):
            if isinstance(node, ast.Import) and any(a.name == "oracle" for a in node.names):
                users.add(fn.name)
    top = [n for n in tree.body if isinstance(n, (ast.Import, ast.ImportFrom))]
    assert not any(isinstance(n, ast.Import) and any(a.name == "oracle" for a in n.names) for n in top)
    assert users <= {"oracle_sample", "run_reference"}, users
